"""GPU parity: the CUDA path (through the C ABI) against the oracle, element by element.

Bar (BASELINE.json north_star): integer graphs bit-exact; fp32 graphs every
element |err| <= 1e-5 * max(1, |ref|).  Sizes span several CTA tiles plus a
ragged tail.  Inputs are seeded (workloads.inputs); input lengths come from the
oracle's own in_items (never from the CUDA path).
"""
import numpy as np
import pytest

from workloads import apps, inputs

pytestmark = pytest.mark.gpu

TOL = 1e-5


def _torch():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    return torch


def run_gpu(prog, x, n, **plan_kw):
    torch = _torch()
    from paper_conf_cgo_nguyenl16_b200 import sg
    with sg.plan(prog, plan_kw.pop("n_gpus", 1), **plan_kw) as p:
        xd = torch.from_numpy(x).cuda()
        dt = torch.int32 if prog.dtype == "i32" else torch.float32
        yd = torch.full((max(1, p.output_items(n)),), -7, dtype=dt, device="cuda")
        p.run(xd, n, yd)
        torch.cuda.synchronize()
        launches = p.last_launch_count()
        return yd[: p.output_items(n)].cpu().numpy(), p.info(), launches


def assert_parity(prog, y, ref):
    assert y.shape == ref.shape, (y.shape, ref.shape)
    if prog.dtype == "i32":
        bad = np.nonzero(y != ref)[0]
        assert bad.size == 0, f"{bad.size} mismatches, first at {bad[:5]}: {y[bad[:5]]} vs {ref[bad[:5]]}"
        return
    err = np.abs(y.astype(np.float64) - ref.astype(np.float64))
    lim = TOL * np.maximum(1.0, np.abs(ref.astype(np.float64)))
    bad = np.nonzero(~(err <= lim))[0]
    assert bad.size == 0, f"{bad.size} elements out of tolerance, first at {bad[:5]}: {y[bad[:5]]} vs {ref[bad[:5]]}"


SMALL = {"bitonic32": 3 * 256 + 17, "fft64": 300, "fmradio10": 1500, "filterbank64": 100, "beamformer12x4": 3}


@pytest.mark.parametrize("name", list(apps.CONFIGS))
def test_parity_small(oracle_lib, name):
    prog = apps.CONFIGS[name]()
    n = SMALL[name]
    x = inputs.make_input(prog.dtype, oracle_lib.in_items(prog, n), inputs.SEEDS[name])
    ref = oracle_lib.run(prog, x, n)
    y, info, launches = run_gpu(prog, x, n)
    assert launches >= 1
    assert_parity(prog, y, ref)


@pytest.mark.parametrize("variant", ["ties", "sorted", "reversed"])
def test_parity_bitonic_variants(oracle_lib, variant):
    prog = apps.bitonic(32)
    n = 1000
    x = inputs.make_input("i32", 32 * n, 5, variant=variant)
    y, _, _ = run_gpu(prog, x, n)
    assert np.array_equal(y, oracle_lib.run(prog, x, n))


@pytest.mark.parametrize("variant", ["impulse", "dc"])
def test_parity_fft_variants(oracle_lib, variant):
    prog = apps.fft(64)
    n = 64
    x = inputs.make_input("f32", 256 * n, 0, variant=variant, block=64)
    y, _, _ = run_gpu(prog, x, n)
    assert_parity(prog, y, oracle_lib.run(prog, x, n))


def test_parity_filterbank_exact_integers(oracle_lib):
    prog = apps.filterbank(64, small_int=True)
    n = 77
    x = inputs.make_input("f32", 8 * n, 3, variant="smallint")
    y, _, _ = run_gpu(prog, x, n)
    assert np.array_equal(y, oracle_lib.run(prog, x, n))


def test_zero_iterations_is_noop():
    torch = _torch()
    from paper_conf_cgo_nguyenl16_b200 import sg
    with sg.plan(apps.bitonic(32), 1) as p:
        y = torch.full((4,), 5, dtype=torch.int32, device="cuda")
        p.run(torch.zeros(4, dtype=torch.int32, device="cuda"), 0, y)
        torch.cuda.synchronize()
        assert y.tolist() == [5, 5, 5, 5]


@pytest.mark.parametrize("n", [1, 2, 255, 256, 257])
def test_parity_bitonic_edge_sizes(oracle_lib, n):
    prog = apps.bitonic(32)
    x = inputs.make_input("i32", 32 * n, n)
    y, _, _ = run_gpu(prog, x, n)
    assert np.array_equal(y, oracle_lib.run(prog, x, n))


# ---- second workloads of the paper's suite: BitonicRec, DCT, MatMul
EXTRA_N = {"bitonicrec32": (3 * 256 + 5, 20000), "dct16": (37, 5000), "matmul16": (41, 5000), "matmul3_16": (29, 3000),
           "des16": (3 * 256 + 5, 20000)}


@pytest.mark.parametrize("name", list(apps.EXTRA))
def test_parity_extra(oracle_lib, name):
    prog = apps.EXTRA[name]()
    for n in EXTRA_N[name]:
        x = inputs.make_input(prog.dtype, oracle_lib.in_items(prog, n), inputs.SEEDS.get(name, 99) + n)
        ref = oracle_lib.run(prog, x, n)
        y, info, launches = run_gpu(prog, x, n)
        assert launches >= 1
        assert_parity(prog, y, ref)


def test_parity_matmul_exact_small_integers(oracle_lib):
    prog = apps.matmul(16, 16, 16)
    n = 300
    rng = np.random.default_rng(8)
    x = rng.integers(-7, 8, size=512 * n).astype(np.float32)
    y, _, _ = run_gpu(prog, x, n)
    assert np.array_equal(y, oracle_lib.run(prog, x, n))


@pytest.mark.parametrize("variant", ["ties", "sorted", "reversed"])
def test_parity_bitonic_rec_variants(oracle_lib, variant):
    prog = apps.bitonic_rec(32)
    n = 1000
    x = inputs.make_input("i32", 32 * n, 6, variant=variant)
    y, _, _ = run_gpu(prog, x, n)
    assert np.array_equal(y, oracle_lib.run(prog, x, n))


# ---- DES (Fig. 4.2a): published known answers through the CUDA path
def test_des_known_answers_gpu():
    import json
    import os
    with open(os.path.join(os.path.dirname(__file__), "golden", "des_kat.json")) as f:
        vec = json.load(f)["vectors"]
    for v in vec:
        k, p, c = (int(v[s], 16) for s in ("key", "plaintext", "ciphertext"))
        for decrypt, src, dst in ((False, p, c), (True, c, p)):
            x = np.array([src >> 32, src & 0xFFFFFFFF] * 300, dtype=np.uint32).view(np.int32)
            y, _, _ = run_gpu(apps.des(16, k, decrypt), x, 300)
            u = y.view(np.uint32)
            assert all(((int(u[2 * i]) << 32) | int(u[2 * i + 1])) == dst for i in range(300)), v["cite"]


@pytest.mark.parametrize("rounds", [1, 2, 16, 20])
def test_des_rounds_vs_oracle(oracle_lib, rounds):
    prog = apps.des(rounds, 0xFEDCBA9876543210)
    n = 2 * 256 + 77
    x = inputs.make_input("i32", oracle_lib.in_items(prog, n), 40 + rounds)
    y, _, _ = run_gpu(prog, x, n)
    assert np.array_equal(y, oracle_lib.run(prog, x, n))


def test_permute_any_dtype(oracle_lib):
    from workloads.spec import Filter, Pipeline, Program
    rng = np.random.default_rng(4)
    for dt in ("f32", "i32"):
        idx = rng.integers(0, 12, size=9).tolist()
        idx2 = rng.integers(0, 9, size=13).tolist()       # 9 -> 13 items: duplicates allowed
        prog = Program("perm", dt, Pipeline([Filter("PERMUTE", [12] + idx), Filter("PERMUTE", [9] + idx2)]))
        n = 1000
        x = inputs.make_input(dt, 12 * n, 77)
        y, _, _ = run_gpu(prog, x, n)
        assert np.array_equal(y, oracle_lib.run(prog, x, n))


@pytest.mark.parametrize("mode", ["staged", "general"])
def test_des_staged_modes(oracle_lib, mode):
    """The shared-memory (staged) code paths on a bit graph: fused roots and the general path with
    runtime PERMUTE readers."""
    prog = apps.des(2, 0x0E329232EA6D0D73)
    n = 700
    x = inputs.make_input("i32", oracle_lib.in_items(prog, n), 91)
    y, _, _ = run_gpu(prog, x, n, codegen_mode=mode)
    assert np.array_equal(y, oracle_lib.run(prog, x, n))


@pytest.mark.parametrize("n", [1, 31, 33, 1023, 1025, 3 * 4096 + 7])
def test_des_bitslice_ragged_and_register_mode(oracle_lib, n):
    """Bitsliced DES (32 iterations per thread, 1024 per warp) on ragged sizes, against the oracle and
    against the thread-per-iteration register kernel."""
    prog = apps.des(16, 0x3B3898371520F75E)
    x = inputs.make_input("i32", oracle_lib.in_items(prog, n), 500 + n)
    ref = oracle_lib.run(prog, x, n)
    y, info, _ = run_gpu(prog, x, n)
    assert np.array_equal(y, ref)
    y2, _, _ = run_gpu(prog, x, n, codegen_mode="register")
    assert np.array_equal(y2, ref)


def test_des_bitslice_misaligned_buffers(oracle_lib):
    """Input / output pointers not 8-byte aligned: the bitsliced kernel's scalar load / store path."""
    torch = _torch()
    from paper_conf_cgo_nguyenl16_b200 import sg
    prog = apps.des(16)
    n = 5000
    x = inputs.make_input("i32", oracle_lib.in_items(prog, n), 321)
    ref = oracle_lib.run(prog, x, n)
    with sg.plan(prog, 1) as p:
        xb = torch.zeros(x.size + 1, dtype=torch.int32, device="cuda")
        xb[1:] = torch.from_numpy(x).cuda()
        yb = torch.full((p.output_items(n) + 1,), -7, dtype=torch.int32, device="cuda")
        p.run(xb[1:], n, yb[1:])
        torch.cuda.synchronize()
        assert np.array_equal(yb[1:].cpu().numpy(), ref)
        assert int(yb[0]) == -7


@pytest.mark.parametrize("name", ["bitonic32", "fmradio10", "filterbank64", "des16", "fft64"])
def test_run_host_chunked_pipeline(oracle_lib, name):
    """sg_run_host with host buffers: single-partition plans pipeline chunks of iterations (copy in /
    kernel / copy out on three streams); every chunk boundary, the stream-start tiles and the input
    prefix each chunk needs must give the oracle's output."""
    _torch()
    from paper_conf_cgo_nguyenl16_b200 import sg
    prog = {**apps.CONFIGS, **apps.EXTRA}[name]()
    n = 4099 if name != "filterbank64" else 2051
    x = inputs.make_input(prog.dtype, oracle_lib.in_items(prog, n), 606)
    ref = oracle_lib.run(prog, x, n)
    with sg.plan(prog, 1) as p:
        y = np.empty(p.output_items(n), dtype=np.int32 if prog.dtype == "i32" else np.float32)
        p.run_host(x, n, y)
    assert_parity(prog, y, ref)


@pytest.mark.parametrize("case", ["beamformer_level_split", "filterbank8_cuts"])
def test_run_host_fragment_pipeline(oracle_lib, case):
    """sg_run_host with a multi-partition one-GPU plan: each fragment's input prefix is copied in and its
    output range out on the host streams, interleaved with the fragment pipeline (the BeamFormer plan is
    the planner's level split; the FilterBank one a user split into three partitions with small
    fragments, so many fragments, copies and ring slots interleave)."""
    _torch()
    from paper_conf_cgo_nguyenl16_b200 import sg
    if case == "beamformer_level_split":
        prog, n, kw = apps.beamformer(), 9, {}
    else:
        prog, n = apps.filterbank(8), 3001
        with sg.plan(prog, 1, plan_only=1) as p0:
            nn = p0.info()["n_nodes"]
        kw = dict(node_partition=[min(2, v * 3 // nn) for v in range(nn)], iters_per_fragment=256)
    x = inputs.make_input(prog.dtype, oracle_lib.in_items(prog, n), 717)
    ref = oracle_lib.run(prog, x, n)
    with sg.plan(prog, 1, **kw) as p:
        assert p.info()["n_partitions"] >= 2
        y = np.empty(p.output_items(n), dtype=np.float32)
        p.run_host(x, n, y)
        y2 = np.empty_like(y)
        p.run_host(x, n, y2)          # a second call reuses the staging buffers and events
    assert_parity(prog, y, ref)
    assert np.array_equal(y, y2)


def test_parity_dct_staged_fused(oracle_lib):
    """2-D DCT in staged mode: the fused path stores through the transposing joins with generated index
    readers over dense buffers (a view map not affine in the store loop)."""
    prog = apps.dct2d(16)
    for n in (37, 3001):
        x = inputs.make_input("f32", 256 * n, 4242 + n)
        ref = oracle_lib.run(prog, x, n)
        y, info, _ = run_gpu(prog, x, n, codegen_mode="staged", partitioner="single")
        assert info["partition_mode"] == [2]
        assert_parity(prog, y, ref)


@pytest.mark.parametrize("G", [2, 4])
def test_parity_gather_partitions(oracle_lib, G):
    """Partitions of views only run as gather kernels (periodic affine copies or generic index chains):
    BeamFormer's channel-to-beam join + duplicate, per-filter splits of FMRadio and FFT."""
    for prog, n in ((apps.beamformer(channels=4, beams=2, frame=64, taps=8, mf_taps=16), 7),
                    (apps.fmradio(5), 900), (apps.fft(16), 500)):
        x = inputs.make_input("f32", oracle_lib.in_items(prog, n), 77 + G)
        ref = oracle_lib.run(prog, x, n)
        y, info, _ = run_gpu(prog, x, n, n_gpus=G, virtual_gpus=1, partitioner="per_filter",
                             iters_per_fragment=max(1, n // 3))
        assert 5 in info["partition_mode"]
        assert_parity(prog, y, ref)


@pytest.mark.parametrize("name", ["dct16", "matmul16", "matmul3_16"])
@pytest.mark.parametrize("runs,vol,db,stage", [("1", "1", "0", "0"), ("2", "0", "0", "0"), ("4", "1", "0", "0"),
                                               ("8", "0", "0", "0"), ("4", "0", "1", "0"), ("8", "1", "1", "0"),
                                               ("4", "0", "0", "1"), ("2", "1", "0", "1")])
def test_demand_runs_parity(oracle_lib, monkeypatch, name, runs, vol, db, stage):
    """Demand-ordered register kernels with K output-group runs per iteration row (K warps share one
    transposed row in shared memory), either input re-read form and single or double-buffered (cp.async)
    tiles: every combination, and a ragged last tile (n not a multiple of the tile's rows), gives the
    oracle's output."""
    _torch()
    monkeypatch.setenv("SG_DEMAND_K", runs)
    monkeypatch.setenv("SG_DEMAND_VOL", vol)
    monkeypatch.setenv("SG_DEMAND_DB", db)
    monkeypatch.setenv("SG_DEMAND_STAGE", stage)
    prog = apps.EXTRA[name]()
    n = 1000 + 37
    x = inputs.make_input(prog.dtype, oracle_lib.in_items(prog, n), 9100 + int(runs))
    ref = oracle_lib.run(prog, x, n)
    y, info, _ = run_gpu(prog, x, n)
    assert info["partition_mode"] == [1]
    assert_parity(prog, y, ref)


@pytest.mark.parametrize("forced", ["1/9,2/13,4/1", "t64x1/5,t64x2/3,t512x1/7"])
def test_beamformer_blockings_parity(oracle_lib, monkeypatch, forced):
    """Sliding-window frame FIRs at blockings the model does not pick (odd B from 1 to 13, paired and
    unpaired), one kernel and the level split: the same outputs as the oracle (the tap order per output
    never changes)."""
    _torch()
    monkeypatch.setenv("SG_BEAM_B", forced)
    prog = apps.beamformer()
    n = 5
    x = inputs.make_input("f32", 24576 * n, 3131)
    ref = oracle_lib.run(prog, x, n)
    for split in ("1", None):
        if split:
            monkeypatch.setenv("SG_NO_LEVEL_SPLIT", split)
        else:
            monkeypatch.delenv("SG_NO_LEVEL_SPLIT", raising=False)
        y, info, _ = run_gpu(prog, x, n)
        if split:
            assert info["n_partitions"] == 1
        assert_parity(prog, y, ref)


@pytest.mark.parametrize("name", ["filterbank64", "filterbank8"])
def test_fir_pairs_ffma2_parity(oracle_lib, name):
    """Opt-in packed sibling FIRs (SG_FIR_FFMA2=1: two accumulators per FFMA2, each lane an IEEE fma in the
    FIR's tap order): the oracle's output.  The variable is read once per process, so the plan is built in
    a subprocess."""
    import os
    import subprocess
    import sys
    _torch()
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    code = ("import sys, numpy as np, torch; sys.path.insert(0, %r)\n"
            "from paper_conf_cgo_nguyenl16_b200 import sg\nfrom workloads import apps, inputs\nfrom oracle import oracle\n"
            "prog = apps.CONFIGS[%r]() if %r in apps.CONFIGS else apps.filterbank(8)\nn = 777\n"
            "x = inputs.make_input('f32', oracle.in_items(prog, n), 4321)\nref = oracle.run(prog, x, n)\n"
            "with sg.plan(prog, 1) as p:\n"
            "    assert '__ffma2_rn' in p.source(0)\n"
            "    xd = torch.from_numpy(x).cuda(); yd = torch.empty(p.output_items(n), device='cuda')\n"
            "    p.run(xd, n, yd); torch.cuda.synchronize(); y = yd.cpu().numpy()\n"
            "err = np.abs(y.astype(np.float64) - ref)\n"
            "assert np.all(err <= 1e-5 * np.maximum(1.0, np.abs(ref)))\nprint('ok')\n") % (root, name, name)
    r = subprocess.run([sys.executable, "-c", code], env=dict(os.environ, SG_FIR_FFMA2="1"), capture_output=True,
                       text=True, timeout=600)
    assert r.returncode == 0 and "ok" in r.stdout, r.stderr[-3000:]


def test_beamformer_ffma2_parity(oracle_lib):
    """Opt-in packed complex MACs of the sliding-window frame FIRs (SG_BEAM_FFMA2=1: (re, im) as one float2,
    two FFMA2 per tap, lane by lane the fmaf sequence of the complex MAC): the oracle's output, in the
    planner's level-split plan.  The variable is read once per process: subprocess."""
    import os
    import subprocess
    import sys
    _torch()
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    code = ("import sys, numpy as np, torch; sys.path.insert(0, %r)\n"
            "from paper_conf_cgo_nguyenl16_b200 import sg\nfrom workloads import apps, inputs\nfrom oracle import oracle\n"
            "prog = apps.beamformer()\nn = 4\n"
            "x = inputs.make_input('f32', oracle.in_items(prog, n), 5151)\nref = oracle.run(prog, x, n)\n"
            "with sg.plan(prog, 1) as p:\n"
            "    assert '__ffma2_rn' in p.source(0) + p.source(p.info()['n_partitions'] - 1)\n"
            "    xd = torch.from_numpy(x).cuda(); yd = torch.empty(p.output_items(n), device='cuda')\n"
            "    p.run(xd, n, yd); torch.cuda.synchronize(); y = yd.cpu().numpy()\n"
            "err = np.abs(y.astype(np.float64) - ref)\n"
            "assert np.all(err <= 1e-5 * np.maximum(1.0, np.abs(ref)))\nprint('ok')\n") % root
    r = subprocess.run([sys.executable, "-c", code], env=dict(os.environ, SG_BEAM_FFMA2="1"), capture_output=True,
                       text=True, timeout=600)
    assert r.returncode == 0 and "ok" in r.stdout, r.stderr[-3000:]
