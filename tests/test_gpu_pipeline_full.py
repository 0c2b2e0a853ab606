"""GPU: the BASELINE multi-GPU configs in their pipelined plans, at full size, on virtual GPUs.

The paper's method maps partitions onto G GPUs and pipelines fragments of iterations through them
(section 3.2.3); fragments are independent given their input window
(PAPER.md:560-561), which is also what makes sampling valid here.  For each BASELINE multi-GPU
config (BASELINE.json configs 3-5) and G, two plans run at the bench size on G virtual GPUs (G
stream pairs of one B200; boundary streams through the double-buffered rings of the one-process
runtime):

* the plan the planner emits (Algorithm 1 + ILP, chain fission considered, replicas = 1), and
* the chain-fission plan with one partition per group.

Each output must be BIT-IDENTICAL to the one-partition output (Kahn determinism; every rewrite is
order-preserving), and sampled windows plus the stream start must match the oracle.
"""
import zlib

import numpy as np
import pytest

from workloads import apps, inputs
from test_gpu_parity import assert_parity

pytestmark = pytest.mark.gpu

N_FULL = {"filterbank64": 1 << 20, "fmradio10": 1 << 24, "beamformer12x4": 4096}
# input items for n iterations (closed forms; the oracle's in_items bisects whole runs)
IN_ITEMS = {"filterbank64": lambda n: 8 * n, "fmradio10": lambda n: 379 + 5 * n, "beamformer12x4": lambda n: 24576 * n}
CASES = [("filterbank64", 2), ("filterbank64", 4), ("filterbank64", 8),
         ("beamformer12x4", 2), ("beamformer12x4", 4), ("fmradio10", 2)]


def _torch():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    return torch


def _run(prog, xd, n, n_gpus, **kw):
    torch = _torch()
    from paper_conf_cgo_nguyenl16_b200 import sg
    with sg.plan(prog, n_gpus, **kw) as p:
        yd = torch.full((p.output_items(n),), -7.0, dtype=torch.float32, device="cuda")
        p.run(xd, n, yd)
        torch.cuda.synchronize()
        return yd.cpu().numpy(), p.info()


def _sampled_vs_oracle(oracle_lib, name, prog, x, y, n):
    rng = np.random.default_rng(zlib.crc32(name.encode()))
    if name == "filterbank64":       # 8 in / 8 out per iteration; FIR memory < 8 iterations
        warm, m = 8, 16
        for s in list(rng.choice(n - m - warm, 12, replace=False)) + [n - m - warm]:
            ref = oracle_lib.run(prog, x[8 * s: 8 * (s + warm + m)], warm + m)[8 * warm:]
            assert_parity(prog, y[8 * (s + warm): 8 * (s + warm + m)], ref)
        assert_parity(prog, y[: 8 * m], oracle_lib.run(prog, x[: 8 * m], m))   # stream start (Delay prework)
    elif name == "fmradio10":        # 5 in / 1 out, 379-item history: a window of input == whole
        m = 64
        for s in list(rng.choice(n - m, 12, replace=False)) + [0, n - m]:
            ref = oracle_lib.run(prog, x[5 * s: 5 * s + 379 + 5 * m], m)
            assert_parity(prog, y[s: s + m], ref)
    else:                            # BeamFormer: frames are independent
        for f in list(rng.choice(n, 4, replace=False)) + [0, n - 1]:
            ref = oracle_lib.run(prog, x[24576 * f: 24576 * (f + 1)], 1)
            assert_parity(prog, y[2048 * f: 2048 * (f + 1)], ref)


@pytest.mark.parametrize("name,G", CASES)
def test_pipelined_plans_full_size(oracle_lib, name, G):
    torch = _torch()
    prog = apps.CONFIGS[name]()
    n = N_FULL[name]
    x = inputs.make_input("f32", IN_ITEMS[name](n), inputs.SEEDS[name])
    xd = torch.from_numpy(x).cuda()
    base, _ = _run(prog, xd, n, 1)
    _sampled_vs_oracle(oracle_lib, name, prog, x, base, n)
    plans = [dict(virtual_gpus=1, replicas=1)]
    if G <= 10:
        plans.append(dict(virtual_gpus=1, replicas=1, chain_groups=G, partitioner="chain"))
    if name == "beamformer12x4":     # no split-join is eligible for fission (no ADD, RR splitter)
        plans = plans[:1]
    for kw in plans:
        y, info = _run(prog, xd, n, G, **kw)
        assert y.tobytes() == base.tobytes(), f"{name} G={G} {kw}: not bit-identical to one partition"
        if kw.get("partitioner") == "chain":
            assert info["chain_fission"] and info["n_partitions"] == G
            assert sorted(info["partition_gpu"]) == list(range(G))
    _sampled_vs_oracle(oracle_lib, name, prog, x, y, n)


@pytest.mark.parametrize("name,G", [("filterbank64", 4), ("fmradio10", 3)])
def test_chain_fission_bit_identical_any_partitioning(oracle_lib, name, G):
    """The fissioned graph itself (forward chain + accumulate chain) under one partition, one per
    filter, and the chain groups with tiny fragments: bit-identical to the graph as written."""
    torch = _torch()
    prog = apps.CONFIGS[name]()
    n = 3001
    x = inputs.make_input("f32", oracle_lib.in_items(prog, n), 5150)
    xd = torch.from_numpy(x).cuda()
    base, _ = _run(prog, xd, n, 1)
    assert_parity(prog, base, oracle_lib.run(prog, x, n))
    for kw, gpus in ((dict(chain_groups=G, partitioner="single"), 1),
                     (dict(chain_groups=G, partitioner="per_filter", iters_per_fragment=500), 1),
                     (dict(chain_groups=G, partitioner="chain", virtual_gpus=1, iters_per_fragment=97), G),
                     (dict(chain_groups=G, partitioner="chain", virtual_gpus=1, iters_per_fragment=211, transport=1), G)):
        y, info = _run(prog, xd, n, gpus, **kw)
        assert info["chain_fission"]
        assert y.tobytes() == base.tobytes(), f"{kw}: not bit-identical"
