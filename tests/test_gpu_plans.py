"""GPU: plan invariance, the multi-GPU fragment pipeline (virtual GPUs on one
B200), random-graph fuzzing, and parity at BASELINE.json's full sizes.

* Plan invariance: every plan of a graph (one partition, one per filter,
  Algorithm 1 for G = 1/2/4, virtual GPUs, tiny fragments that cycle the
  double-buffered rings) gives BIT-IDENTICAL output (Kahn determinism; all
  rewrites are order-preserving), equal to the oracle.
* Full sizes, in the launch configuration bench.py times: outputs checked on
  sampled iterations the oracle computes one window at a time (iterations are
  independent given their input window), plus properties at any size
  (Bitonic: every row sorted and a permutation of its input row).
"""
import numpy as np
import pytest

from workloads import apps, inputs
from test_gpu_parity import assert_parity, run_gpu

pytestmark = pytest.mark.gpu


def _torch():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    return torch


PLANS = [
    dict(partitioner="single"),
    dict(partitioner="per_filter", iters_per_fragment=96),
    dict(n_gpus=2, virtual_gpus=1, iters_per_fragment=128),
    dict(n_gpus=4, virtual_gpus=1, iters_per_fragment=64),
    dict(n_gpus=3, virtual_gpus=1, partitioner="per_filter", iters_per_fragment=200),
    # hybrid replica x pipeline plans: fragments dealt round-robin to groups
    dict(n_gpus=4, virtual_gpus=1, replicas=2, iters_per_fragment=64),
    dict(n_gpus=4, virtual_gpus=1, replicas=4, iters_per_fragment=50),
    dict(n_gpus=6, virtual_gpus=1, replicas=3, partitioner="per_filter", iters_per_fragment=70),
    # transports (include/sg.h): cudaMemcpyPeerAsync for every cut edge even between virtual GPUs of one
    # device, and the host-staged D2H + H2D pair of [7]
    dict(n_gpus=3, virtual_gpus=1, partitioner="per_filter", iters_per_fragment=90, transport=1),
    dict(n_gpus=2, virtual_gpus=1, partitioner="per_filter", iters_per_fragment=150, transport=2),
]


@pytest.mark.parametrize("name,prog_fn,n", [
    ("fmradio3", lambda: apps.fmradio(4), 900),
    ("filterbank8", lambda: apps.filterbank(8), 500),
    ("bitonic8", lambda: apps.bitonic(8), 1000),
    ("fft16", lambda: apps.fft(16), 700),
    ("des3", lambda: apps.des(3), 700),
    ("beamformer_small", lambda: apps.beamformer(channels=3, beams=2, frame=64, taps=8, mf_taps=16), 9),
])
def test_plan_invariance(oracle_lib, name, prog_fn, n):
    _torch()
    prog = prog_fn()
    x = inputs.make_input(prog.dtype, oracle_lib.in_items(prog, n), 1234)
    ref = oracle_lib.run(prog, x, n)
    outs = []
    for kw in PLANS:
        y, info, launches = run_gpu(prog, x, n, **dict(kw))
        assert_parity(prog, y, ref)
        outs.append((kw, y, info))
    base = outs[0][1]
    for kw, y, info in outs[1:]:
        assert y.tobytes() == base.tobytes(), f"plan {kw} not bit-identical"


@pytest.mark.parametrize("seed", range(16))
def test_random_graphs_vs_oracle(oracle_lib, seed):
    _torch()
    prog = apps.random_program(seed, "f32" if seed % 2 else "i32")
    n = 300
    x = inputs.make_input(prog.dtype, oracle_lib.in_items(prog, n), seed)
    ref = oracle_lib.run(prog, x, n)
    for kw in (dict(partitioner="single"), dict(partitioner="per_filter", iters_per_fragment=64),
               dict(n_gpus=2, virtual_gpus=1, iters_per_fragment=50)):
        y, _, _ = run_gpu(prog, x, n, **kw)
        assert_parity(prog, y, ref)


def test_multi_gpu_plan_uses_several_gpus():
    _torch()
    from paper_conf_cgo_nguyenl16_b200 import sg
    with sg.plan(apps.filterbank(64), 4, virtual_gpus=1) as p:
        i = p.info()
        assert i["n_partitions"] >= 2
        assert len(set(i["partition_gpu"])) >= 2
        assert i["ilp_optimal"]


# ---------------------------------------------------------------- full size
def test_bitonic_full_size_properties():
    torch = _torch()
    from paper_conf_cgo_nguyenl16_b200 import sg
    n = 1 << 20
    x = inputs.make_input("i32", 32 * n, inputs.SEEDS["bitonic32"])
    with sg.plan(apps.bitonic(32), 1) as p:
        xd = torch.from_numpy(x).cuda()
        yd = torch.empty_like(xd)
        p.run(xd, n, yd)
        torch.cuda.synchronize()
        ref = torch.sort(xd.view(n, 32), dim=1).values
        assert torch.equal(yd.view(n, 32), ref)       # sorted + permutation of each row


def test_fft_full_size_sampled(oracle_lib):
    torch = _torch()
    from paper_conf_cgo_nguyenl16_b200 import sg
    prog = apps.fft(64)
    n = 1 << 20
    x = inputs.make_input("f32", 256 * n, inputs.SEEDS["fft64"])
    with sg.plan(prog, 1) as p:
        xd = torch.from_numpy(x).cuda()
        yd = torch.empty_like(xd)
        p.run(xd, n, yd)
        torch.cuda.synchronize()
        y = yd.cpu().numpy()
    rng = np.random.default_rng(7)
    for k in list(rng.choice(n, 200, replace=False)) + [0, n - 1]:
        ref = oracle_lib.run(prog, x[256 * k: 256 * (k + 1)], 1)
        assert_parity(prog, y[256 * k: 256 * (k + 1)], ref)


def test_fmradio_full_size_sampled(oracle_lib):
    torch = _torch()
    from paper_conf_cgo_nguyenl16_b200 import sg
    prog = apps.fmradio(11)
    n = 1 << 24
    x = inputs.make_input("f32", 379 + 5 * n, inputs.SEEDS["fmradio10"])
    with sg.plan(prog, 1) as p:
        xd = torch.from_numpy(x).cuda()
        yd = torch.empty(n, dtype=torch.float32, device="cuda")
        p.run(xd, n, yd)
        torch.cuda.synchronize()
        y = yd.cpu().numpy()
    rng = np.random.default_rng(8)
    m = 64
    for s in list(rng.choice(n - m, 40, replace=False)) + [0, n - m]:
        ref = oracle_lib.run(prog, x[5 * s: 5 * s + 379 + 5 * m], m)   # peeking graph: window == whole
        assert_parity(prog, y[s: s + m], ref)


def test_filterbank_full_size_sampled(oracle_lib):
    torch = _torch()
    from paper_conf_cgo_nguyenl16_b200 import sg
    prog = apps.filterbank(64)
    n = 1 << 20
    x = inputs.make_input("f32", 8 * n, inputs.SEEDS["filterbank64"])
    with sg.plan(prog, 1) as p:
        xd = torch.from_numpy(x).cuda()
        yd = torch.empty(8 * n, dtype=torch.float32, device="cuda")
        p.run(xd, n, yd)
        torch.cuda.synchronize()
        y = yd.cpu().numpy()
    rng = np.random.default_rng(9)
    warm, m = 8, 16
    for s in list(rng.choice(n - m - warm, 20, replace=False)) + [n - m - warm]:
        ref = oracle_lib.run(prog, x[8 * s: 8 * (s + warm + m)], warm + m)[8 * warm:]
        assert_parity(prog, y[8 * (s + warm): 8 * (s + warm + m)], ref)
    assert_parity(prog, y[: 8 * m], oracle_lib.run(prog, x[: 8 * m], m))   # stream start (Delay prework)


def test_beamformer_full_size_sampled(oracle_lib):
    torch = _torch()
    from paper_conf_cgo_nguyenl16_b200 import sg
    prog = apps.beamformer()
    n = 4096
    x = inputs.make_input("f32", 24576 * n, inputs.SEEDS["beamformer12x4"])
    with sg.plan(prog, 1) as p:
        xd = torch.from_numpy(x).cuda()
        yd = torch.empty(2048 * n, dtype=torch.float32, device="cuda")
        p.run(xd, n, yd)
        torch.cuda.synchronize()
        y = yd.cpu().numpy()
    rng = np.random.default_rng(10)
    for f in list(rng.choice(n, 6, replace=False)) + [0, n - 1]:
        ref = oracle_lib.run(prog, x[24576 * f: 24576 * (f + 1)], 1)
        assert_parity(prog, y[2048 * f: 2048 * (f + 1)], ref)


def test_run_rank_world1_nccl(oracle_lib):
    """sg_run_rank through an NCCL communicator of one rank (the one-process-per-GPU path);
    per-filter partitions exercise the local rings and event ordering of sg_dist.cpp."""
    torch = _torch()
    import os
    import torch.distributed as dist
    from paper_conf_cgo_nguyenl16_b200 import sg
    from paper_conf_cgo_nguyenl16_b200.dist import pipeline_plan
    created = not dist.is_initialized()
    if created:
        os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
        os.environ.setdefault("MASTER_PORT", "29517")
        dist.init_process_group("nccl", rank=0, world_size=1, device_id=torch.device("cuda", 0))
    try:
        prog = apps.fmradio(4)
        n = 2000
        x = inputs.make_input("f32", oracle_lib.in_items(prog, n), 77)
        ref = oracle_lib.run(prog, x, n)
        for kw in (dict(), dict(partitioner="per_filter", iters_per_fragment=300)):
            p = pipeline_plan(prog, **kw)
            xd = torch.from_numpy(x).cuda()
            yd = torch.empty(p.output_items(n), device="cuda")
            p.run_rank(xd, n, yd)
            torch.cuda.synchronize()
            assert_parity(prog, yd.cpu().numpy(), ref)
            p.close()
    finally:
        if created:
            dist.destroy_process_group()



@pytest.mark.parametrize("name", ["filterbank64", "fmradio10", "beamformer12x4", "des16"])
def test_hybrid_auto_plan_vs_oracle(oracle_lib, name):
    """replicas = -1: the cost model picks R; whatever it picks, the output is the oracle's."""
    _torch()
    prog = {**apps.CONFIGS, **apps.EXTRA}[name]()
    n = 9 if name == "beamformer12x4" else 3000
    x = inputs.make_input(prog.dtype, oracle_lib.in_items(prog, n), 4321)
    ref = oracle_lib.run(prog, x, n)
    y, info, launches = run_gpu(prog, x, n, n_gpus=8, virtual_gpus=1, replicas=-1,
                                iters_per_fragment=1 if name == "beamformer12x4" else 200)
    assert_parity(prog, y, ref)
    assert info["replicas"] >= 1 and 8 % info["replicas"] == 0


def test_des_full_size_sampled(oracle_lib):
    """DES at the bench size (2^22 blocks, bitsliced, rolled rounds): sampled blocks against the oracle
    one by one, plus a published known-answer block planted at both ends of the stream."""
    torch = _torch()
    from paper_conf_cgo_nguyenl16_b200 import sg
    prog = apps.des(16)
    n = 1 << 22
    x = inputs.make_input("i32", 2 * n, inputs.SEEDS["des16"])
    kat_p, kat_c = 0x0123456789ABCDEF, 0x85E813540F0AB405      # Grabbe's worked example (default key)
    for k in (0, n - 1):
        x[2 * k: 2 * k + 2] = np.array([kat_p >> 32, kat_p & 0xFFFFFFFF], dtype=np.uint32).view(np.int32)
    with sg.plan(prog, 1) as p:
        xd = torch.from_numpy(x).cuda()
        yd = torch.empty_like(xd)
        p.run(xd, n, yd)
        torch.cuda.synchronize()
        y = yd.cpu().numpy()
    for k in (0, n - 1):
        u = y[2 * k: 2 * k + 2].view(np.uint32)
        assert (int(u[0]) << 32 | int(u[1])) == kat_c
    rng = np.random.default_rng(11)
    ks = np.sort(rng.choice(n, 300, replace=False))
    blocks = np.concatenate([x[2 * k: 2 * k + 2] for k in ks])
    ref = oracle_lib.run(prog, blocks, len(ks))
    got = np.concatenate([y[2 * k: 2 * k + 2] for k in ks])
    assert np.array_equal(got, ref)


@pytest.mark.parametrize("name,n", [("fmradio10", 1 << 20), ("beamformer12x4", 256), ("dct16", 1 << 16)])
def test_profile_partitions_measures_the_kernels(name, n):
    """sg_profile_partitions (the measured side of the PEE validation, Fig. 4.1 analog): one positive time per
    partition, and their sum agrees with the plan's own run of the same iterations on one GPU (partitions
    run back to back there) within a factor that allows for the zero-filled streams and launch overheads."""
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_cgo_nguyenl16_b200 import sg
    prog = {**apps.CONFIGS, **apps.EXTRA}[name]()
    with sg.plan(prog, 1) as p:
        t = p.profile_partitions(n, reps=3)
        assert len(t) == p.info()["n_partitions"] and all(x > 0 for x in t)
        x = torch.zeros(p.input_items(n), dtype=torch.float32, device="cuda")
        y = torch.empty(p.output_items(n), dtype=torch.float32, device="cuda")
        p.run(x, n, y)
        torch.cuda.synchronize()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        for _ in range(3):
            p.run(x, n, y)
        e1.record()
        torch.cuda.synchronize()
        run_ns = e0.elapsed_time(e1) / 3 * 1e6 / n
        assert 0.5 < sum(t) / run_ns < 2.0, (t, run_ns)
