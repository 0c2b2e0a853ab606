"""Pins for the oracle (oracle/sg_oracle.c) against things other than itself.

Each pin is chosen so that a plausible mistake in the oracle (a dropped term, a
wrong sign or index, a transposed operand, a wrong rate) fails at least one:

  rates        closed-form repetition vectors of the five programs (derived by
               hand from their structure), the balance
               equations on random graphs, the empirical output/input ratio,
               an inconsistent graph rejected
  FFT          numpy double FFT within 10*log2(N)*2^-24; impulse -> twiddles;
               DC -> N at bin 0; exactly one splitter and one joiner
               
  Bitonic      numpy sort (ties, sorted, reversed, full-range keys)
  FIR          direct convolution: exact on small integers, Higham bound otherwise
  FilterBank   multirate identity y = sum_b F_b * up(down(H_b * delay(x))):
               exact on small integers, bounded on the benchmark coefficients
  FMRadio      components (LPF = convolution, demod closed form, band = hi - lo) and end to end
               within a rigorous float32 error bound around a float64 evaluation
               and an end-to-end numpy double reference within a loose bound
  BeamFormer   numpy complex convolution / mat-vec / abs per frame
  Kahn         two schedules and three chunk sizes give bit-identical output
  windows      a run started mid-stream equals the whole run after the memory
  in_items     minimal input prefixes: closed forms
"""
import math

import numpy as np
import pytest

from workloads import apps, inputs
from workloads.spec import Filter, Pipeline, Program, SplitJoin

U = 2.0 ** -24


def gamma(n):
    return n * U / (1 - n * U)


# --------------------------------------------------------------------- rates
def test_rates_fft_closed_form(oracle_lib):
    r = oracle_lib.rates(apps.fft(64))
    assert r["in_per_iter"] == 256 and r["out_per_iter"] == 256
    kinds = r["kind"]
    for k, rep, pop in zip(kinds, r["reps"], r["pop"]):
        if k == 6:      # FFT_REORDER(n): pop 2n, fires 64/n per iteration
            assert rep == 64 // (pop // 2)
        elif k == 7:    # COMBINE_DFT(j): fires 64/j
            assert rep == 64 // (pop // 2)
        else:           # the one splitter and the one joiner
            assert rep == 1
    assert sum(1 for t in r["type"] if t != 0) == 2


def test_rates_bitonic_closed_form(oracle_lib):
    r = oracle_lib.rates(apps.bitonic(32))
    assert len(r["reps"]) == 368
    for t, rep, pop, push in zip(r["type"], r["reps"], r["pop"], r["push"]):
        if t == 0:
            assert rep == 1                   # every CompareExchange fires once
        elif t == 2:   # step splitter RR(L) x numseq pops 32 -> once; PBS splitter RR(1) x L/2 gets L -> twice
            assert rep == (1 if pop == 32 else 2)
        elif t == 3:
            assert rep == (1 if push == 32 else 2)
    assert r["in_per_iter"] == r["out_per_iter"] == 32


def test_rates_fmradio_all_once(oracle_lib):
    r = oracle_lib.rates(apps.fmradio(11))
    assert len(r["reps"]) == 65
    assert set(r["reps"]) == {1}
    assert r["in_per_iter"] == 5 and r["out_per_iter"] == 1


def test_rates_filterbank_closed_form(oracle_lib):
    r = oracle_lib.rates(apps.filterbank(64))
    assert len(r["reps"]) == 387
    want = {2: 8, 1: 8, 3: 1, 4: 1, 11: 8}   # DELAY, FIR, DECIMATE, EXPAND, ADD
    for t, k, rep in zip(r["type"], r["kind"], r["reps"]):
        if t == 0:
            assert rep == want[k]
        else:
            assert rep == 8                   # dup splitter and RR(1) joiner
    assert r["in_per_iter"] == 8 and r["out_per_iter"] == 8


def test_rates_beamformer_closed_form(oracle_lib):
    r = oracle_lib.rates(apps.beamformer())
    got = list(zip(r["type"], r["kind"], r["reps"]))
    assert got[0] == (2, -1, 1024)                   # split RR(2) x 12: 24 floats per firing
    for t, k, rep in got[1:25]:
        assert (t, k, rep) == (0, 12, 1)             # one frame per FIR
    assert got[25] == (3, -1, 512)                   # join RR(2) x 12
    assert got[26] == (1, -1, 12288)                 # dup splitter, 1 item per firing
    beams = got[27:39]
    for b in range(4):
        assert [x[2] for x in beams[3 * b: 3 * b + 3]] == [512, 1, 512]
    assert got[39] == (3, -1, 512)
    assert r["in_per_iter"] == 24576 and r["out_per_iter"] == 2048


def _edge_list(prog):
    """(producer push, consumer pop) per edge, walking the spec independently."""
    edges = []

    def build(s, prod):  # prod = (node_idx, push) of the producer feeding s
        if isinstance(s, Filter):
            pop, push = _filter_pop_push(s)
            me = len(nodes)
            nodes.append(s)
            if prod is not None:
                edges.append((prod[0], prod[1], me, pop))
            return (me, push)
        if isinstance(s, Pipeline):
            p = prod
            for c in s.children:
                p = build(c, p)
            return p
        nb = len(s.branches)
        me = len(nodes)
        nodes.append(("split", s))
        tot = 1 if s.split == "dup" else sum(s.split_w)
        if prod is not None:
            edges.append((prod[0], prod[1], me, tot))
        outs = []
        for b in range(nb):
            w = 1 if s.split == "dup" else s.split_w[b]
            outs.append(build(s.branches[b], (me, w)))
        j = len(nodes)
        nodes.append(("join", s))
        for b in range(nb):
            edges.append((outs[b][0], outs[b][1], j, s.join_w[b]))
        return (j, sum(s.join_w))

    nodes = []
    build(prog.top, None)
    return edges


def _filter_pop_push(f):
    k, iv = f.kind, f.ints
    return {
        "IDENTITY": (1, 1), "FIR": (iv[1], 1) if f.kind == "FIR" else None, "DELAY": (1, 1),
        "DECIMATE": (iv[0], 1) if iv else None, "EXPAND": (1, iv[0]) if iv else None,
        "COMPARE_EXCHANGE": (2, 2), "FFT_REORDER": (2 * iv[0], 2 * iv[0]) if iv else None,
        "COMBINE_DFT": (2 * iv[0], 2 * iv[0]) if iv else None, "FM_DEMOD": (1, 1), "SUBTRACT": (2, 1),
        "AMPLIFY": (1, 1), "ADD": (iv[0], 1) if iv else None,
        "BEAM_FIR": (2 * iv[2], 2 * iv[2] // iv[1]) if len(iv) >= 3 else None,
        "BEAMFORM": (2 * iv[0], 2) if iv else None, "MAGNITUDE": (2, 1), "MULTIPLY": (2, 1),
    }[k]


@pytest.mark.parametrize("seed", range(40))
def test_rates_balance_random(oracle_lib, seed):
    prog = apps.random_program(seed, "f32" if seed % 2 else "i32")
    r = oracle_lib.rates(prog)
    reps = r["reps"]
    assert math.gcd(*reps) == 1 if len(reps) > 1 else reps[0] == 1
    for (u, push, v, pop) in _edge_list(prog):
        assert reps[u] * push == reps[v] * pop


@pytest.mark.parametrize("name", list(apps.CONFIGS))
def test_rates_match_empirical_ratio(oracle_lib, name):
    prog = apps.CONFIGS[name]()
    r = oracle_lib.rates(prog)
    n = 4 if name == "beamformer12x4" else 64
    L = oracle_lib.in_items(prog, n) + 3 * r["in_per_iter"]
    x = np.zeros(L, np.int32 if prog.dtype == "i32" else np.float32)
    y = oracle_lib.run_items(prog, x, 10 ** 9)
    assert y.size == (n + 3) * r["out_per_iter"]


def test_inconsistent_graph_rejected(oracle_lib):
    bad = Program("bad", "f32", Pipeline([SplitJoin("dup", [Filter("IDENTITY"), Filter("DECIMATE", [2])])]))
    with pytest.raises(oracle_lib.OracleError) as e:
        oracle_lib.rates(bad)
    assert e.value.code == -3


# ----------------------------------------------------------------------- FFT
def _fft_rows(x, n_iters, N=64):
    c = x.reshape(n_iters, 2, N, 2).astype(np.float64)
    return c[..., 0] + 1j * c[..., 1]


def test_fft_vs_numpy(oracle_lib):
    prog = apps.fft(64)
    n = 64
    x = inputs.make_input("f32", 256 * n, 0xF0F1)
    y = oracle_lib.run(prog, x, n)
    Z = np.fft.fft(_fft_rows(x, n), axis=-1)
    Y = _fft_rows(y, n)
    for it in range(n):
        for b in range(2):
            err = np.linalg.norm(Y[it, b] - Z[it, b]) / np.linalg.norm(Z[it, b])
            assert err <= 10 * 6 * U


def test_fft_impulse_gives_twiddles(oracle_lib):
    prog = apps.fft(64)
    x = inputs.make_input("f32", 256 * 4, 0, variant="impulse", block=64)
    Y = _fft_rows(oracle_lib.run(prog, x, 4), 4)
    k = np.arange(64)
    ref = np.exp(-2j * np.pi * k / 64)
    assert np.max(np.abs(Y - ref)) < 4e-7 * 6


def test_fft_dc(oracle_lib):
    prog = apps.fft(64)
    x = inputs.make_input("f32", 256 * 2, 0, variant="dc")
    Y = _fft_rows(oracle_lib.run(prog, x, 2), 2)
    assert np.all(Y[..., 0] == 64)
    assert np.max(np.abs(Y[..., 1:])) < 1e-5


def test_fft_has_one_splitter_one_joiner():
    # "FFT only has one splitter and one joiner" (chapter V)
    c = apps.fft(64).count_nodes()
    assert c == {"filters": 22, "splitters": 1, "joiners": 1}


@pytest.mark.parametrize("N", [8, 16, 128])
def test_fft_other_sizes(oracle_lib, N):
    prog = apps.fft(N)
    x = inputs.make_input("f32", 4 * N * 3, 7)
    y = oracle_lib.run(prog, x, 3)
    Z = np.fft.fft(_fft_rows(x, 3, N), axis=-1)
    Y = _fft_rows(y, 3, N)
    assert np.linalg.norm(Y - Z) / np.linalg.norm(Z) <= 10 * math.log2(N) * U


# ------------------------------------------------------------------- Bitonic
@pytest.mark.parametrize("variant", ["uniform", "ties", "sorted", "reversed"])
def test_bitonic_sorts(oracle_lib, variant):
    prog = apps.bitonic(32)
    x = inputs.make_input("i32", 32 * 500, 0xB170, variant=variant)
    y = oracle_lib.run(prog, x, 500)
    assert np.array_equal(y.reshape(-1, 32), np.sort(x.reshape(-1, 32), axis=1))


@pytest.mark.parametrize("N", [4, 8, 16, 64])
def test_bitonic_other_sizes(oracle_lib, N):
    prog = apps.bitonic(N)
    x = inputs.make_input("i32", N * 100, N)
    y = oracle_lib.run(prog, x, 100)
    assert np.array_equal(y.reshape(-1, N), np.sort(x.reshape(-1, N), axis=1))


def test_bitonic_node_count():
    assert apps.bitonic(32).count_nodes() == {"filters": 240, "splitters": 64, "joiners": 64}


# ----------------------------------------------------------------------- FIR
def _direct_fir(x, c, pop, n_out):
    L = len(c)
    return np.array([sum(float(x[g * pop + i]) * float(c[i]) for i in range(L)) for g in range(n_out)])


@pytest.mark.parametrize("L,pop", [(1, 1), (5, 1), (8, 3), (2, 4), (32, 1), (64, 5)])
def test_fir_exact_small_integers(oracle_lib, L, pop):
    c = [float((i * 7) % 5 - 2) for i in range(L)]
    prog = Program("fir", "f32", Pipeline([Filter("FIR", [L, pop], c)]))
    x = inputs.make_input("f32", 400, 3, variant="smallint")
    n_out = (400 - max(L, pop)) // pop + 1
    y = oracle_lib.run_items(prog, x, 10 ** 6)
    assert y.size == n_out
    assert np.array_equal(y.astype(np.float64), _direct_fir(x, c, pop, n_out))


def test_fir_higham_bound(oracle_lib):
    L = 64
    c = apps.lowpass_coeffs(250e6, 108e6, L)
    prog = Program("fir", "f32", Pipeline([Filter("FIR", [L, 5], c)]))
    x = inputs.make_input("f32", 5000, 9)
    y = oracle_lib.run_items(prog, x, 10 ** 6)
    n_out = (5000 - L) // 5 + 1
    ref = _direct_fir(x, c, 5, n_out)
    bound = gamma(L) * np.array([sum(abs(float(x[g * 5 + i]) * c[i]) for i in range(L)) for g in range(n_out)])
    assert np.all(np.abs(y - ref) <= bound)


# ---------------------------------------------------------------- FilterBank
def _filterbank_numpy(x, branches, M=8, L=32, small_int=False, absval=False):
    """Textbook multirate filter bank in float64: sum_b F_b * up_M(down_M(H_b * delay(x)))."""
    x = np.abs(x).astype(np.float64) if absval else x.astype(np.float64)
    n = x.size
    total = np.zeros(n)
    for b in range(branches):
        H = np.array([i * 32 + b * 64 + 2 * b + i + 1 for i in range(L)], np.float64)
        F = np.array([i * b + b * b + b + i for i in range(L)], np.float64)
        if small_int:
            H, F = (H % 5) - 2, (F % 5) - 2
        if absval:
            H, F = np.abs(H), np.abs(F)
        d1 = np.concatenate([np.zeros(L - 1), x])
        h = np.array([np.dot(d1[g:g + L], H[::-1]) for g in range(n)])   # sum peek(i) * H[L-1-i]
        e = np.zeros(n)
        e[::M] = h[::M]                                                    # down then up
        d2 = np.concatenate([np.zeros(L - 1), e])
        f = np.array([np.dot(d2[g:g + L], F[::-1]) for g in range(n)])
        total += f
    return total


def test_filterbank_exact_small_integers(oracle_lib):
    prog = apps.filterbank(8, small_int=True)
    n = 40
    x = inputs.make_input("f32", 8 * n, 5, variant="smallint")
    y = oracle_lib.run(prog, x, n)
    ref = _filterbank_numpy(x, 8, small_int=True)
    assert np.array_equal(y.astype(np.float64), ref)


def test_filterbank_bounded(oracle_lib):
    prog = apps.filterbank(16)
    n = 32
    x = inputs.make_input("f32", 8 * n, 0xFB64)
    y = oracle_lib.run(prog, x, n)
    ref = _filterbank_numpy(x, 16)
    A = _filterbank_numpy(x, 16, absval=True)
    assert np.all(np.abs(y - ref) <= 200 * U * A + 1e-30)


# ------------------------------------------------------------------- FMRadio
def test_fm_demod_closed_form(oracle_lib):
    prog = Program("demod", "f32", Pipeline([Filter("FM_DEMOD", [], [2.0e8])]))
    x = inputs.make_input("f32", 1000, 11)
    y = oracle_lib.run_items(prog, x, 10 ** 6)
    p = (x[:-1] * x[1:]).astype(np.float32).astype(np.float64)       # x0*x1 in float
    ref = (np.float64(np.float32(2.0e8)) * np.arctan(p)).astype(np.float32)
    ulp = np.spacing(np.abs(ref))
    assert y.size == 999 and np.all(np.abs(y - ref) <= ulp)


def test_bandpass_is_difference_of_lowpasses(oracle_lib):
    lo, hi = apps.lowpass_coeffs(250e6, 55.0, 64), apps.lowpass_coeffs(250e6, 110.0, 64)
    prog = Program("bpf", "f32", Pipeline([SplitJoin("dup", [Filter("FIR", [64, 1], lo), Filter("FIR", [64, 1], hi)]),
                                            Filter("SUBTRACT")]))
    x = inputs.make_input("f32", 500, 12)
    y = oracle_lib.run_items(prog, x, 10 ** 6)
    a = oracle_lib.run_items(Program("a", "f32", Pipeline([Filter("FIR", [64, 1], lo)])), x, 10 ** 6)
    b = oracle_lib.run_items(Program("b", "f32", Pipeline([Filter("FIR", [64, 1], hi)])), x, 10 ** 6)
    assert np.array_equal(y, (b - a).astype(np.float32))               # x1 - x0: high minus low


def _fmradio_numpy(x, n, bands=11, taps=64):
    rate, cutoff, decim = 250e6, 108e6, 4
    c1 = np.array(apps.lowpass_coeffs(rate, cutoff, taps), np.float64)
    m = 379 + 5 * n
    x = x[:m].astype(np.float64)
    n1 = n + 64
    l1 = np.array([np.dot(x[5 * g:5 * g + taps], c1) for g in range(n1)])
    gain = 27000.0 * (rate / (10000.0 * math.pi))
    dm = gain * np.arctan(l1[:-1] * l1[1:])
    cut = [math.exp(i * (math.log(1760.0) - math.log(55.0)) / (bands - 1) + math.log(55.0)) for i in range(bands)]
    out = np.zeros(n)
    for i in range(1, bands):
        lo = np.array(apps.lowpass_coeffs(rate, cut[i - 1], taps), np.float64)
        hi = np.array(apps.lowpass_coeffs(rate, cut[i], taps), np.float64)
        val = ((i - 1) - (bands - 2) / 2.0) / 5.0
        g = 2.0 - val if val > 0 else 2.0 + val
        band = np.array([np.dot(dm[k:k + taps], hi) - np.dot(dm[k:k + taps], lo) for k in range(n)])
        out += np.float64(np.float32(g)) * band
    return out


def test_fmradio_end_to_end_loose(oracle_lib):
    # Structural pin: a dropped band, a swapped subtraction or a wrong tap index
    # gives O(1) relative error; float32 vs float64 evaluation differs by far less.
    prog = apps.fmradio(11)
    n = 200
    x = inputs.make_input("f32", 379 + 5 * n, 0xF3, variant="fmtone")
    y = oracle_lib.run(prog, x, n).astype(np.float64)
    ref = _fmradio_numpy(x, n)
    assert np.linalg.norm(y - ref) / np.linalg.norm(ref) < 2e-3


def _fmradio_bound(x, n, bands=11, taps=64, drop_band=None):
    """FMRadio in float64 plus a rigorous elementwise bound on the float32 evaluation's error (Higham:
    a length-L FMA dot product is within gamma_L * sum|c||x| of the exact one; the product and the
    1-Lipschitz atan propagate first-order terms; every later rounding adds a unit roundoff)."""
    u = 2.0 ** -24
    gam = lambda k: k * u / (1 - k * u)
    rate, cutoff = 250e6, 108e6
    c1 = np.array(apps.lowpass_coeffs(rate, cutoff, taps), np.float64)
    x = x[:379 + 5 * n].astype(np.float64)
    X = np.array([x[5 * g:5 * g + taps] for g in range(n + 64)])
    l1, e1 = X @ c1, gam(taps) * (np.abs(X) @ np.abs(c1))
    a, b, ea, eb = l1[:-1], l1[1:], e1[:-1], e1[1:]
    p = a * b
    ep = np.abs(a) * eb + np.abs(b) * ea + ea * eb + u * (np.abs(p) + np.abs(a) * eb + np.abs(b) * ea + ea * eb)
    gain = np.float64(np.float32(27000.0 * (rate / (10000.0 * math.pi))))
    dm = gain * np.arctan(p)
    edm = gain * ep + 2 * u * np.abs(dm) + 1e-14 * np.abs(dm)
    cut = [math.exp(i * (math.log(1760.0) - math.log(55.0)) / (bands - 1) + math.log(55.0)) for i in range(bands)]
    D = np.array([dm[k:k + taps] for k in range(n)])
    ED = np.array([edm[k:k + taps] for k in range(n)])
    out, err = np.zeros(n), np.zeros(n)
    for i in range(1, bands):
        lo = np.array(apps.lowpass_coeffs(rate, cut[i - 1], taps), np.float64)
        hi = np.array(apps.lowpass_coeffs(rate, cut[i], taps), np.float64)
        val = ((i - 1) - (bands - 2) / 2.0) / 5.0
        g = np.float64(np.float32(2.0 - val if val > 0 else 2.0 + val))
        band = D @ hi - D @ lo
        eh = gam(taps) * (np.abs(D) @ np.abs(hi)) + ED @ np.abs(hi)
        el = gam(taps) * (np.abs(D) @ np.abs(lo)) + ED @ np.abs(lo)
        eband = eh + el + u * (np.abs(band) + eh + el)
        if i != drop_band:
            out += g * band
        err += g * eband + u * (g * np.abs(band) + g * eband)
    err += gam(bands - 1) * (np.abs(out) + err)
    return out, err


@pytest.mark.parametrize("variant", ["fmtone", "uniform"])
def test_fmradio_end_to_end_within_error_bound(oracle_lib, variant):
    """FMRadio end to end, pinned elementwise by the float32 error bound of _fmradio_bound; the same
    bound rejects a dropped band (negative control), so the pin is discriminating."""
    prog = apps.fmradio(11)
    n = 300
    x = inputs.make_input("f32", 379 + 5 * n, 0xF3, variant=variant)
    y = oracle_lib.run(prog, x, n).astype(np.float64)
    ref, err = _fmradio_bound(x, n)
    assert np.all(np.abs(y - ref) <= err)
    bad, _ = _fmradio_bound(x, n, drop_band=5)
    assert np.sum(np.abs(y - bad) > err) > n // 2


# ---------------------------------------------------------------- BeamFormer
def _beamformer_numpy(x, frames, ch=12, beams=4, frame=1024, taps=64, mf=512):
    def w(L):
        return np.array([(math.sin(i + 1) + 1j * math.cos(i + 1)) / (i + 1) for i in range(L)])
    w1, wmf = w(taps), w(mf)
    out = np.zeros((frames, frame // 2, beams))
    xs = x.reshape(frames, frame, ch, 2).astype(np.float64)
    for f in range(frames):
        z = xs[f, :, :, 0] + 1j * xs[f, :, :, 1]                  # [t, c]
        a = np.stack([np.convolve(z[:, c], w1)[:frame] for c in range(ch)], axis=1)
        b = np.stack([np.convolve(a[:, c], w1)[:frame][::2] for c in range(ch)], axis=1)  # dec 2
        for bb in range(beams):
            wb = np.array([(math.sin(c + 1) + 1j * math.cos(c + 1)) / (bb + c + 1) for c in range(ch)])
            s = b @ wb
            m = np.convolve(s, wmf)[: frame // 2]
            out[f, :, bb] = np.abs(m)
    return out.reshape(-1)


def test_beamformer_vs_numpy(oracle_lib):
    prog = apps.beamformer()
    frames = 2
    x = inputs.make_input("f32", 24576 * frames, 0xBEA3)
    y = oracle_lib.run(prog, x, frames).astype(np.float64)
    ref = _beamformer_numpy(x, frames)
    assert np.max(np.abs(y - ref) / np.maximum(1.0, np.abs(ref))) < 1e-4
    # frames are independent: permuting input frames permutes output frames
    xp = np.concatenate([x[24576:], x[:24576]])
    yp = oracle_lib.run(prog, xp, frames)
    assert np.array_equal(yp[:2048], y[2048:].astype(np.float32))


# --------------------------------------------------------- Kahn determinism
@pytest.mark.parametrize("name", list(apps.CONFIGS))
def test_kahn_determinism_configs(oracle_lib, name):
    prog = apps.CONFIGS[name]()
    r = oracle_lib.rates(prog)
    n = 2 if name == "beamformer12x4" else 40
    L = oracle_lib.in_items(prog, n)
    x = inputs.make_input(prog.dtype, L, 99)
    base = oracle_lib.run(prog, x, n)
    for chunk, order in [(1 if r["in_per_iter"] < 100 else 97, 0), (17, 1), (1 << 20, 1)]:
        y = oracle_lib.run(prog, x, n, chunk=chunk, order_seed=order)
        assert y.tobytes() == base.tobytes()


@pytest.mark.parametrize("seed", range(20))
def test_kahn_determinism_random(oracle_lib, seed):
    prog = apps.random_program(seed, "f32" if seed % 2 else "i32")
    x = inputs.make_input(prog.dtype, 3000, seed)
    a = oracle_lib.run_items(prog, x, 10 ** 7, chunk=4096, order_seed=0)
    b = oracle_lib.run_items(prog, x, 10 ** 7, chunk=7, order_seed=1)
    assert a.tobytes() == b.tobytes()


# ------------------------------------------------------- windows / in_items
def test_window_equals_whole_fmradio(oracle_lib):
    prog = apps.fmradio(11)
    n, s = 120, 37
    x = inputs.make_input("f32", 379 + 5 * n, 0xF3)
    whole = oracle_lib.run(prog, x, n)
    part = oracle_lib.run(prog, x[5 * s:], n - s)    # pure peeking graph: no warm-up needed
    assert part.tobytes() == whole[s:].tobytes()


def test_window_equals_whole_filterbank_after_memory(oracle_lib):
    prog = apps.filterbank(64)
    n, s, warm = 64, 20, 8
    x = inputs.make_input("f32", 8 * n, 0xFB64)
    whole = oracle_lib.run(prog, x, n)
    part = oracle_lib.run(prog, x[8 * s:], n - s)
    assert part[8 * warm:].tobytes() == whole[8 * (s + warm):].tobytes()
    assert part[:8].tobytes() != whole[8 * s:8 * s + 8].tobytes()     # Delay history is real


@pytest.mark.parametrize("name,form", [("fft64", lambda n: 256 * n), ("bitonic32", lambda n: 32 * n),
                                       ("fmradio10", lambda n: 379 + 5 * n), ("filterbank64", lambda n: 8 * n),
                                       ("beamformer12x4", lambda n: 24576 * n)])
def test_in_items_closed_forms(oracle_lib, name, form):
    prog = apps.CONFIGS[name]()
    for n in (1, 2, 7):
        assert oracle_lib.in_items(prog, n) == form(n)
