"""Pins for the oracle on the second workloads of the paper's suite (
Fig. 4.2 d/e/f/g): BitonicRec, DCT and MatMul.

  BitonicRec  numpy sort per block (full-range keys, ties, sorted, reversed blocks);
              every CompareExchange fires once per iteration
  DCT         scipy's orthonormal 2-D DCT-II in double within two stacked Higham
              bounds; a constant block has only its DC coefficient (= N * value);
              the transform is orthonormal (Parseval, within the bound)
  MatMul      numpy double product within gamma_K * |A||B|; bit-exact on small
              integers (every product and partial sum is an integer < 2^24);
              identity and permutation matrices reproduce / permute A
  MULTIPLY    a one-filter graph against the float32 product
"""
import numpy as np
import pytest
import scipy.fft

from workloads import apps, inputs
from workloads.spec import Filter, Pipeline, Program

U = 2.0 ** -24


def gamma(n):
    return n * U / (1 - n * U)


# ---------------------------------------------------------------- BitonicRec
@pytest.mark.parametrize("variant", ["uniform", "ties", "sorted", "reversed"])
def test_bitonic_rec_sorts(oracle_lib, variant):
    prog = apps.bitonic_rec(32)
    n = 300
    x = inputs.make_input("i32", 32 * n, 11, variant=variant)
    y = oracle_lib.run(prog, x, n)
    assert np.array_equal(y.reshape(n, 32), np.sort(x.reshape(n, 32), axis=1))


@pytest.mark.parametrize("N", [2, 4, 8, 16, 64])
def test_bitonic_rec_other_sizes(oracle_lib, N):
    prog = apps.bitonic_rec(N)
    n = 40
    x = inputs.make_input("i32", N * n, N)
    assert np.array_equal(oracle_lib.run(prog, x, n).reshape(n, N), np.sort(x.reshape(n, N), axis=1))


def test_bitonic_rec_rates(oracle_lib):
    r = oracle_lib.rates(apps.bitonic_rec(32))
    assert r["in_per_iter"] == 32 and r["out_per_iter"] == 32
    # N log2(N) (log2(N) + 1) / 4 compare-exchanges, each fires once per iteration
    ce = [rep for t, k, rep in zip(r["type"], r["kind"], r["reps"]) if t == 0]
    assert len(ce) == 32 * 5 * 6 // 4 and all(rep == 1 for rep in ce)


# ----------------------------------------------------------------------- DCT
def _dct_ref(x, N):
    return scipy.fft.dctn(x.astype(np.float64).reshape(N, N), type=2, norm="ortho")


@pytest.mark.parametrize("N", [4, 8, 16])
def test_dct_vs_scipy(oracle_lib, N):
    prog = apps.dct2d(N)
    n = 12
    x = inputs.make_input("f32", N * N * n, 21 + N)
    y = oracle_lib.run(prog, x, n).reshape(n, N, N).astype(np.float64)
    C = np.array(apps.dct_coeffs(N), dtype=np.float64)
    for i in range(n):
        X = x[i * N * N:(i + 1) * N * N].astype(np.float64).reshape(N, N)
        ref = _dct_ref(X, N)
        # rounding of the f32 coefficients (|dC| <= U |C|) plus two dot-product stages
        bound = (gamma(N) + 2 * U) * (np.abs(C) @ np.abs(X) @ np.abs(C).T) * 3 + 1e-30
        assert np.all(np.abs(y[i] - ref) <= bound), (i, np.max(np.abs(y[i] - ref) / bound))


def test_dct_constant_block_is_dc_only(oracle_lib):
    N = 16
    prog = apps.dct2d(N)
    x = np.full(N * N * 2, 0.5, np.float32)
    y = oracle_lib.run(prog, x, 2).reshape(2, N, N).astype(np.float64)
    assert abs(y[0, 0, 0] - 0.5 * N) <= 1e-5 * N
    y[:, 0, 0] = 0
    assert np.max(np.abs(y)) <= 1e-5


def test_dct_parseval(oracle_lib):
    N = 16
    prog = apps.dct2d(N)
    x = inputs.make_input("f32", N * N * 4, 5)
    y = oracle_lib.run(prog, x, 4).astype(np.float64).reshape(4, -1)
    e_in = np.sum(x.astype(np.float64).reshape(4, -1) ** 2, axis=1)
    assert np.allclose(np.sum(y ** 2, axis=1), e_in, rtol=1e-5)


# -------------------------------------------------------------------- MatMul
def _mm_blocks(x, M, K, N, n):
    blocks = []
    for i in range(n):
        base = i * (M * K + K * N)
        A = x[base:base + M * K].astype(np.float64).reshape(M, K)
        B = x[base + M * K:base + M * K + K * N].astype(np.float64).reshape(K, N)
        blocks.append((A, B))
    return blocks


@pytest.mark.parametrize("M,K,N", [(16, 16, 16), (3, 5, 7), (8, 1, 4), (1, 9, 2)])
def test_matmul_vs_numpy(oracle_lib, M, K, N):
    prog = apps.matmul(M, K, N)
    n = 6
    x = inputs.make_input("f32", (M * K + K * N) * n, M * 100 + K * 10 + N)
    y = oracle_lib.run(prog, x, n).reshape(n, M, N).astype(np.float64)
    for i, (A, B) in enumerate(_mm_blocks(x, M, K, N, n)):
        bound = gamma(K) * (np.abs(A) @ np.abs(B)) + 1e-30
        assert np.all(np.abs(y[i] - A @ B) <= bound)


def test_matmul_exact_small_integers(oracle_lib):
    M, K, N = 16, 16, 16
    prog = apps.matmul(M, K, N)
    n = 5
    rng = np.random.default_rng(3)
    x = rng.integers(-7, 8, size=(M * K + K * N) * n).astype(np.float32)
    y = oracle_lib.run(prog, x, n).reshape(n, M, N)
    for i, (A, B) in enumerate(_mm_blocks(x, M, K, N, n)):
        assert np.array_equal(y[i], (A @ B).astype(np.float32))


def test_matmul_identity_and_permutation(oracle_lib):
    M = K = N = 8
    prog = apps.matmul(M, K, N)
    A = inputs.make_input("f32", M * K, 9).reshape(M, K)
    P = np.eye(N, dtype=np.float32)[::-1]                    # reverses the columns of A
    x = np.concatenate([A.ravel(), np.eye(K, dtype=np.float32).ravel(), A.ravel(), P.ravel()])
    y = oracle_lib.run(prog, x, 2).reshape(2, M, N)
    assert np.array_equal(y[0], A)
    assert np.array_equal(y[1], A[:, ::-1])


@pytest.mark.parametrize("M,K,N,D", [(16, 16, 16, 4), (3, 6, 5, 2), (4, 8, 2, 8)])
def test_matmul3_vs_numpy(oracle_lib, M, K, N, D):
    """MatMul3 (blocked): each of the D block dot products within gamma(K/D), their sum within one more
    gamma(D) -- bounded by gamma(K/D + D) |A| |B|."""
    prog = apps.matmul_block(M, K, N, D)
    n = 5
    x = inputs.make_input("f32", (M * K + K * N) * n, M * 1000 + K * 100 + N * 10 + D)
    y = oracle_lib.run(prog, x, n).reshape(n, M, N).astype(np.float64)
    for i, (A, B) in enumerate(_mm_blocks(x, M, K, N, n)):
        bound = gamma(K // D + D) * (np.abs(A) @ np.abs(B)) + 1e-30
        assert np.all(np.abs(y[i] - A @ B) <= bound)


def test_matmul3_exact_small_integers_and_block_order(oracle_lib):
    """Exact on small integers; and with D = 1 the blocked graph is MatMul2 bit for bit (same order)."""
    M, K, N = 16, 16, 16
    n = 4
    rng = np.random.default_rng(31)
    x = rng.integers(-7, 8, size=(M * K + K * N) * n).astype(np.float32)
    y = oracle_lib.run(apps.matmul_block(M, K, N, 4), x, n).reshape(n, M, N)
    for i, (A, B) in enumerate(_mm_blocks(x, M, K, N, n)):
        assert np.array_equal(y[i], (A @ B).astype(np.float32))
    xf = inputs.make_input("f32", (M * K + K * N) * n, 5)
    assert oracle_lib.run(apps.matmul_block(M, K, N, 1), xf, n).tobytes() == oracle_lib.run(
        apps.matmul(M, K, N), xf, n).tobytes()


def test_multiply_is_float32_product(oracle_lib):
    prog = Program("mul", "f32", Pipeline([Filter("MULTIPLY")]))
    x = inputs.make_input("f32", 2 * 1000, 4)
    y = oracle_lib.run(prog, x, 1000)
    assert np.array_equal(y, x[0::2] * x[1::2])


@pytest.mark.parametrize("name", list(apps.EXTRA))
def test_extra_kahn_determinism(oracle_lib, name):
    prog = apps.EXTRA[name]()
    n = 9
    x = inputs.make_input(prog.dtype, oracle_lib.in_items(prog, n), 77)
    a = oracle_lib.run(prog, x, n)
    b = oracle_lib.run(prog, x, n, chunk=7, order_seed=3)     # another valid schedule
    assert a.tobytes() == b.tobytes()
