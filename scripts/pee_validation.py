#!/usr/bin/env python
"""PEE validation -- the B200 analog of Fig. 4.1 ("estimated vs
measured partition time").  For every benchmark program and G = 1, 2, 4, 8 (virtual
GPUs on one device), plan with Algorithm 1 + the ILP, then compare each partition's
PEE estimate (sg_plan_info.partition_time, ns/iteration) with its kernel time
measured alone (sg_profile_partitions).  Writes a JSON list and a markdown summary.

    python scripts/pee_validation.py [--out profiles/pee_validation_r01] [--configs a,b]
"""
import argparse
import json
import math
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

# iterations per measurement: enough work to fill the GPU (>= ~1 ms for the heavy graphs)
N_ITERS = {"bitonic32": 1 << 20, "fft64": 1 << 18, "fmradio10": 1 << 22, "filterbank64": 1 << 20,
           "beamformer12x4": 1024, "des16": 1 << 22, "bitonicrec32": 1 << 20, "dct16": 1 << 18, "matmul16": 1 << 18}


def r2(xs, ys):
    mx, my = sum(xs) / len(xs), sum(ys) / len(ys)
    sxx = sum((x - mx) ** 2 for x in xs)
    syy = sum((y - my) ** 2 for y in ys)
    sxy = sum((x - mx) * (y - my) for x, y in zip(xs, ys))
    return (sxy * sxy / (sxx * syy)) if sxx > 0 and syy > 0 else float("nan")


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--out", default=os.path.join(ROOT, "profiles", "pee_validation_r01"))
    ap.add_argument("--configs", default=",".join(N_ITERS))
    ap.add_argument("--gpus", default="1,2,4,8")
    ap.add_argument("--reps", type=int, default=5)
    args = ap.parse_args()
    import torch
    from paper_conf_cgo_nguyenl16_b200 import sg
    from workloads import apps
    assert torch.cuda.is_available()
    rows = []
    for name in args.configs.split(","):
        prog = {**apps.CONFIGS, **apps.EXTRA}[name]()
        for G in [int(g) for g in args.gpus.split(",")]:
            with sg.plan(prog, G, devices=[0] * G) as p:
                info = p.info()
                meas = p.profile_partitions(N_ITERS[name], args.reps)
                for k in range(info["n_partitions"]):
                    nodes = sum(1 for q in info["node_partition"] if q == k)
                    rows.append({"config": name, "G": G, "partition": k, "nodes": nodes,
                                 "gpu": info["partition_gpu"][k], "mode": info["partition_mode"][k],
                                 "est_ns_per_iter": info["partition_time"][k], "meas_ns_per_iter": meas[k]})
                    print(json.dumps(rows[-1]), flush=True)
    with open(args.out + ".json", "w") as f:
        json.dump(rows, f, indent=1)
    est = [r["est_ns_per_iter"] for r in rows]
    mea = [r["meas_ns_per_iter"] for r in rows]
    le, lm = [math.log(x) for x in est], [math.log(y) for y in mea]
    ratios = sorted(m / e for e, m in zip(est, mea))
    lines = ["# PEE validation (Fig. 4.1 analog), %d partitions" % len(rows), "",
             "Estimated (`sg_plan_info.partition_time`) vs measured (`sg_profile_partitions`, kernel alone, "
             "CUDA events, %d reps after a warm-up) ns per iteration, every partition Algorithm 1 + ILP emit for "
             "G = %s (virtual GPUs on one B200)." % (args.reps, args.gpus), "",
             "* R^2 (linear): %.3f" % r2(est, mea),
             "* R^2 (log-log): %.3f" % r2(le, lm),
             "* measured / estimated: median %.2f, min %.2f, max %.2f" % (
                 ratios[len(ratios) // 2], ratios[0], ratios[-1]), "",
             "| config | G | part | nodes | mode | est ns/iter | meas ns/iter | meas/est |", "|---|---|---|---|---|---|---|---|"]
    for r in rows:
        lines.append("| %s | %d | %d | %d | %d | %.4g | %.4g | %.2f |" % (
            r["config"], r["G"], r["partition"], r["nodes"], r["mode"], r["est_ns_per_iter"], r["meas_ns_per_iter"],
            r["meas_ns_per_iter"] / r["est_ns_per_iter"]))
    open(args.out + ".md", "w").write("\n".join(lines) + "\n")
    print("\n".join(lines[:8]))


if __name__ == "__main__":
    main()
