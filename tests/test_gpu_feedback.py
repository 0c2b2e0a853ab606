"""GPU parity of feedback loops against the oracle.

A feedback loop runs as a sequential partition of its own (its state crosses fragments and launches);
the parts around it stay data-parallel.  Every plan -- one GPU, per-filter partitions, virtual GPUs,
tiny fragments that force many state hand-overs and history re-emissions -- must give the oracle's
bytes (integer programs) or stay within the north-star tolerance (fp32)."""
import numpy as np
import pytest

from workloads import apps, inputs
from workloads.spec import FeedbackLoop, Filter, Pipeline, Program

from test_gpu_parity import assert_parity, run_gpu

pytestmark = pytest.mark.gpu

PROGS = {
    "runsum": lambda: Program("rsum", "i32", Pipeline([FeedbackLoop(Filter("ADD", [2]), Filter("IDENTITY"), [1, 1],
                                                                    "dup", enqueue=[0])])),
    "echo64": apps.FEEDBACK["echo64"],           # wavefront of 64 firings (2 warps)
    "echo300": lambda: apps.echo(300, -0.75, 8),  # wavefront capped at 256 firings
    # multi-warp wavefronts that are not powers of two: ring / history slots are shared between lanes
    # of different warps, so the per-step barrier must stay (lane-local chains would race)
    "echo96": lambda: apps.echo(96, 0.5, 8),
    "echo100": lambda: apps.echo(100, -0.5, 8),
    "runstats": apps.FEEDBACK["runstats"],
    "multirate": lambda: Program("mr", "f32", Pipeline([
        Filter("FIR", [5, 1], [0.5, -1.0, 0.25, 2.0, -0.5]),
        FeedbackLoop(Pipeline([Filter("FIR", [3, 3], [0.5, -2.0, 0.25]), Filter("EXPAND", [2])]),
                     Pipeline([Filter("EXPAND", [2]), Filter("DECIMATE", [2]), Filter("DELAY", [3])]), [2, 1], "rr", [1, 1],
                     enqueue=[0.0]),
        Filter("FIR", [4, 3], [1.0, 0.5, 0.25, 0.125])])),
}
PLANS = [dict(), dict(partitioner="per_filter", iters_per_fragment=37),
         dict(n_gpus=2, virtual_gpus=1, iters_per_fragment=64), dict(n_gpus=3, virtual_gpus=1, iters_per_fragment=5)]


@pytest.mark.parametrize("name", list(PROGS))
@pytest.mark.parametrize("plan", range(len(PLANS)))
def test_feedback_parity(oracle_lib, name, plan):
    prog = PROGS[name]()
    n = 1200
    x = inputs.make_input(prog.dtype, oracle_lib.in_items(prog, n), 77)
    ref = oracle_lib.run(prog, x, n)
    y, info, launches = run_gpu(prog, x, n, **dict(PLANS[plan]))
    assert 4 in info["partition_mode"]
    assert_parity(prog, y, ref)


def test_feedback_state_resets_between_runs(oracle_lib):
    """Two sg_run calls on one plan both start from the enqueued items (no state leaks across calls)."""
    import torch
    from paper_conf_cgo_nguyenl16_b200 import sg
    prog = PROGS["runsum"]()
    n = 5000
    x = inputs.make_input("i32", n, 3)
    ref = oracle_lib.run(prog, x, n)
    with sg.plan(prog, 1) as p:
        xd = torch.from_numpy(x).cuda()
        for _ in range(2):
            yd = torch.empty(n, dtype=torch.int32, device="cuda")
            p.run(xd, n, yd)
            torch.cuda.synchronize()
            assert np.array_equal(yd.cpu().numpy(), ref)


@pytest.mark.parametrize("name", ["echo64", "echo96", "runsum"])
@pytest.mark.parametrize("frag", [0, 10000])
def test_feedback_parity_long(oracle_lib, name, frag):
    """n = 2^16 + 37 iterations: long enough that the guard-free interior trips (g1 - gs >= 2*PD*WB
    firings) and the trip-to-trip prefetch refill run, as one fragment and as ~10k-iteration fragments
    (state and history handed over between launches)."""
    prog = PROGS[name]()
    n = (1 << 16) + 37
    x = inputs.make_input(prog.dtype, oracle_lib.in_items(prog, n), 91)
    ref = oracle_lib.run(prog, x, n)
    kw = dict(partitioner="per_filter", iters_per_fragment=frag) if frag else dict()
    y, info, launches = run_gpu(prog, x, n, **kw)
    assert 4 in info["partition_mode"]
    assert_parity(prog, y, ref)
