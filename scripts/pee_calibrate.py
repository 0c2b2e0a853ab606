#!/usr/bin/env python
"""Partition timing corpus for the B200 PEE (the paper calibrates its model constants by regression
over measured partitions, Fig. 4.1 at 705-722).

For a fixed, deterministic set of plans (whole graphs, Algorithm 1 at G = 2/4/8, chain-fission
groups, one partition per filter, random graphs), every partition's kernel is timed alone
(sg_profile_partitions: CUDA events, kernel only) and written with the plan's options and its
node -> partition map, so the features of each partition can be recomputed offline.

    python scripts/pee_calibrate.py --out profiles/pee_corpus_r02.json      # on the GPU box
    python scripts/pee_calibrate.py --compile-only                          # fill the cubin cache (CPU)
"""
import argparse
import json
import os
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

N_ITERS = {"bitonic32": 1 << 20, "fft64": 1 << 18, "fmradio10": 1 << 22, "filterbank64": 1 << 20,
           "beamformer12x4": 1024, "des16": 1 << 22, "bitonicrec32": 1 << 20, "dct16": 1 << 18,
           "matmul16": 1 << 18, "filterbank8": 1 << 21, "fmradio4": 1 << 22}


def corpus():
    """(config name, n_gpus, plan kwargs) -- deterministic plans (the ILP runs on a node budget)."""
    out = []
    for name in ("bitonic32", "fft64", "fmradio10", "filterbank64", "beamformer12x4", "des16", "bitonicrec32",
                 "dct16", "matmul16"):
        out.append((name, 1, {}))
    for name in ("fft64", "fmradio10", "filterbank64", "beamformer12x4"):
        for G in (2, 4, 8):
            out.append((name, G, dict(replicas=1, chain_groups=-1)))
    for name in ("fmradio10", "filterbank64"):
        for G in (2, 4, 8):
            out.append((name, G, dict(replicas=1, chain_groups=G, partitioner="chain")))
    # Algorithm 1 with only the G-aware cap on the graph as written (the round-1 planner's plans)
    for name in ("fmradio10", "filterbank64", "fft64"):
        for G in (2, 4, 8):
            out.append((name, G, dict(replicas=1, chain_groups=-1, env_caps="1")))
    # naive branch splits of the filter bank (the cut the paper's PDG rule prices)
    for G in (2, 4, 8):
        part = [0] * 387
        for b in range(64):
            for k in range(6):
                part[1 + 6 * b + k] = b * G // 64
        part[385] = part[386] = G - 1
        out.append(("filterbank64", G, dict(node_partition=part)))
    out.append(("filterbank8", 1, dict(partitioner="per_filter")))
    out.append(("fmradio4", 1, dict(partitioner="per_filter")))
    out.append(("fft64", 1, dict(partitioner="per_filter")))
    for seed in range(6):
        out.append((f"random{seed}", 1, dict(partitioner="per_filter")))
        out.append((f"random{seed}", 1, dict(partitioner="single")))
    return out


def program(name):
    from workloads import apps
    if name.startswith("random"):
        return apps.random_program(500 + int(name[6:]), "f32" if int(name[6:]) % 2 else "i32")
    extra = {"filterbank8": lambda: apps.filterbank(8), "fmradio4": lambda: apps.fmradio(4)}
    return {**apps.CONFIGS, **apps.EXTRA, **extra}[name]()


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--out", default=os.path.join(ROOT, "profiles", "pee_corpus_r02.json"))
    ap.add_argument("--compile-only", action="store_true")
    ap.add_argument("--reps", type=int, default=5)
    args = ap.parse_args()
    from paper_conf_cgo_nguyenl16_b200 import sg
    rows = []
    for name, G, kw in corpus():
        prog = program(name)
        t0 = time.time()
        kw2 = dict(kw)
        if G > 1:
            kw2["virtual_gpus"] = 1
        caps = kw2.pop("env_caps", None)
        if caps:
            os.environ["SG_A1_CAPS"] = caps
        else:
            os.environ.pop("SG_A1_CAPS", None)
        with sg.plan(prog, G, **kw2) as p:
            info = p.info()
            if args.compile_only:
                print(f"[compile] {name} G={G} {kw}: {info['n_partitions']} partitions, {time.time() - t0:.1f}s", flush=True)
                continue
            n = N_ITERS.get(name, 1 << 18)
            meas = p.profile_partitions(n, args.reps)
            rows.append({"config": name, "G": G, "kw": kw, "n_iters": n, "node_partition": info["node_partition"],
                         "partition_gpu": info["partition_gpu"], "mode": info["partition_mode"],
                         "est_ns_per_iter": info["partition_time"], "meas_ns_per_iter": meas,
                         "chain_fission": info["chain_fission"]})
            print(json.dumps({k: rows[-1][k] for k in ("config", "G", "kw", "mode", "meas_ns_per_iter")}), flush=True)
    if not args.compile_only:
        with open(args.out, "w") as f:
            json.dump(rows, f)


if __name__ == "__main__":
    main()
