#!/usr/bin/env python
"""Small instances of every kernel family, each checked against the oracle -- the workload that
compute-sanitizer (memcheck / racecheck / synccheck) runs over (scripts/sanitize.sh,
tests/test_gpu_sanitize.py).

    python scripts/sanitize_cases.py [--case NAME ...]     (no argument: every case)

Families: TMA register rows (BitonicSort), bulk-copy in-place components (FFT), staged fused with
prefetch (FMRadio, FilterBank), staged general path, bitslice with rolled rounds (DES), feedback loops
(lane-local wavefront and the per-step-barrier wavefront), multi-fragment rings on virtual GPUs
(per-filter partitions and chain fission), frame FIRs (BeamFormer), demand-ordered register rows (DCT),
gather kernels of partitions of views only.
"""
import argparse
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)


def cases():
    from workloads import apps
    return {
        "tma_register": (lambda: apps.bitonic(32), 1100, {}),
        "bulk_components": (lambda: apps.fft(64), 300, {}),
        "staged_fused_fm": (lambda: apps.fmradio(4), 700, {}),
        "staged_fused_fb": (lambda: apps.filterbank(8), 600, {}),
        "staged_general": (lambda: apps.fmradio(3), 400, dict(codegen_mode="general")),
        "bitslice_rolled": (lambda: apps.des(16), 2100, {}),
        "loop_lane_local": (lambda: apps.echo(64), 1500, {}),
        "loop_barrier": (lambda: apps.echo(96, 0.5, 8), 1500, {}),
        "rings_per_filter": (lambda: apps.filterbank(4), 700, dict(n_gpus=3, virtual_gpus=1, partitioner="per_filter",
                                                                   iters_per_fragment=128)),
        "rings_chain": (lambda: apps.filterbank(8), 900, dict(n_gpus=2, virtual_gpus=1, chain_groups=2,
                                                              partitioner="chain", iters_per_fragment=200)),
        "frame_fir": (lambda: apps.beamformer(channels=3, beams=2, frame=64, taps=8, mf_taps=16), 5, {}),
        "demand_register": (lambda: apps.dct2d(16), 300, dict(partitioner="single")),
        "gather_views": (lambda: apps.fmradio(4), 600, dict(partitioner="per_filter", iters_per_fragment=150)),
    }


def run_case(name):
    import numpy as np
    import torch
    from oracle import oracle
    from paper_conf_cgo_nguyenl16_b200 import sg
    from workloads import inputs
    mk, n, kw = cases()[name]
    prog = mk()
    kw = dict(kw)
    x = inputs.make_input(prog.dtype, oracle.in_items(prog, n), 99)
    ref = oracle.run(prog, x, n)
    with sg.plan(prog, kw.pop("n_gpus", 1), **kw) as p:
        xd = torch.from_numpy(x).cuda()
        dt = torch.int32 if prog.dtype == "i32" else torch.float32
        yd = torch.empty(p.output_items(n), dtype=dt, device="cuda")
        p.run(xd, n, yd)
        torch.cuda.synchronize()
        y = yd.cpu().numpy()
    if prog.dtype == "i32":
        ok = np.array_equal(y, ref)
    else:
        ok = bool(np.all(np.abs(y.astype(np.float64) - ref) <= 1e-5 * np.maximum(1.0, np.abs(ref))))
    print(f"[sanitize-case] {name}: {'parity OK' if ok else 'PARITY FAIL'}", flush=True)
    return ok


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--case", nargs="*", default=None)
    args = ap.parse_args()
    names = args.case or list(cases())
    ok = all([run_case(c) for c in names])
    return 0 if ok else 1


if __name__ == "__main__":
    sys.exit(main())
