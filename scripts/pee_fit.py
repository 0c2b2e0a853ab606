#!/usr/bin/env python
"""Fit the B200 PEE's constants to the measured partition corpus (scripts/pee_calibrate.py), the way
the paper calibrates C1, C2 by regression over measured partitions, and report the
Fig. 4.1 analog: R^2 of estimated vs measured partition time.

    python scripts/pee_fit.py profiles/pee_corpus_r02.json [--fit] [--out profiles/pee_validation_r02]

Features come from the plan itself (sg_pee_features: the code generator's pruned / CSE'd work per
iteration); the corpus rows carry the plan options and the node -> partition map, which are checked
against a fresh plan_only plan.  Without --fit the current estimates (sg_plan_info.partition_time) are
evaluated; with --fit the staged-mode constants are refitted (least squares on log time) and printed.
"""
import argparse
import json
import math
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "scripts"))


def features(rows, plan_only=0):
    from paper_conf_cgo_nguyenl16_b200 import sg
    from pee_calibrate import program
    out = []
    for r in rows:
        kw = dict(r["kw"])
        caps = kw.pop("env_caps", None)
        if caps:
            os.environ["SG_A1_CAPS"] = caps
        else:
            os.environ.pop("SG_A1_CAPS", None)
        if r["G"] > 1:
            kw["virtual_gpus"] = 1
        kw["node_partition"] = r["node_partition"]   # exactly the measured partitions
        kw.pop("partitioner", None)
        if r.get("chain_fission") and kw.get("chain_groups", 0) < 2:
            kw["chain_groups"] = r["G"]        # the planner fissions into G / replicas = G groups
        with sg.plan(program(r["config"]), r["G"], plan_only=plan_only, **kw) as p:
            info = p.info()
            for k in range(info["n_partitions"]):
                f = p.pee_features(k)
                # the estimate of a kernel run alone over n iterations: steady state + one launch (ramp, tail)
                f.update(config=r["config"], G=r["G"], kw=r["kw"], part=k, meas=r["meas_ns_per_iter"][k],
                         est_steady=info["partition_time"][k], n=r["n_iters"],
                         est=info["partition_time"][k] + LAUNCH_NS / r["n_iters"],
                         nodes=sum(1 for q in info["node_partition"] if q == k))
                out.append(f)
    os.environ.pop("SG_A1_CAPS", None)
    return out


def r2(xs, ys):
    mx, my = sum(xs) / len(xs), sum(ys) / len(ys)
    sxx = sum((x - mx) ** 2 for x in xs)
    syy = sum((y - my) ** 2 for y in ys)
    sxy = sum((x - mx) * (y - my) for x, y in zip(xs, ys))
    return (sxy * sxy / (sxx * syy)) if sxx > 0 and syy > 0 else float("nan")


LAUNCH_NS = 8.5e3  # sg_plan.cpp kLaunch: one kernel launch including ramp-up and tail

# staged-mode model (sg_plan.cpp pee_estimate), all times in ns per iteration
FP32 = 148 * 128 * 2 * 1.9e9
HBM = 6.5536e12
TILE = 64.0


def staged_model(th, f):
    eff, eff_frame, lvl, smem, fixed = th
    e = eff_frame if f["frame"] else eff
    rec = 1.0 + f["halo_firings"] / (TILE * max(1.0, f["firings"]))
    tc = (f["flops"] / (FP32 * e) + f["dfma"] * 80.0 / 37e12) * rec * 1e9 + smem * (f["reads"] + f["writes"]) / (
        148 * 1.9e9) * 1e9 + lvl * f["levels"] / TILE * 1e9
    tdt = (f["in_bytes"] + f["out_bytes"]) / HBM * 1e9
    return max(tc, tdt) + fixed


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("corpus")
    ap.add_argument("--fit", action="store_true")
    ap.add_argument("--out", default="")
    ap.add_argument("--fit-frame", action="store_true",
                    help="report the e_frame (sg_plan.cpp kModel) that centres the frame-FIR partitions' "
                         "measured / estimated ratio at 1 (geometric mean), given their par_eff")
    args = ap.parse_args()
    rows = json.load(open(args.corpus))
    F = features(rows)
    F = [f for f in F if f["meas"] > 0]
    if args.fit:
        import numpy as np
        from scipy.optimize import least_squares
        S = [f for f in F if f["mode"] == 2]
        x0 = np.array([0.6, 0.3, 1e-9, 0.0, 0.0])

        def res(th):
            return [math.log(staged_model(th, f)) - math.log(f["meas"]) for f in S]
        sol = least_squares(res, x0, bounds=([0.05, 0.05, 0.0, 0.0, 0.0], [1.0, 1.0, 1e-6, 1.0, 1.0]))
        print("fitted staged constants (eff, eff_frame, level s, smem cycles/item, fixed ns):", list(sol.x))
        for f in S:
            f["fit"] = staged_model(sol.x, f)
    if args.fit_frame:
        fr = [f for f in F if f["frame"] and f["mode"] == 2]
        if fr:
            g = math.exp(sum(math.log(f["meas"] / f["est"]) for f in fr) / len(fr))
            print("frame partitions: %d, geometric-mean measured / estimated %.3f -> e_frame x %.3f" % (len(fr), g, 1 / g))
            for f in fr:
                print("  %s G=%d part %d par_eff %.3f est %.1f meas %.1f" % (f["config"], f["G"], f["part"],
                                                                           f.get("par_eff", 1), f["est"], f["meas"]))
    est = [f["est"] for f in F]
    mea = [f["meas"] for f in F]
    ratios = sorted(m / e for e, m in zip(est, mea))
    lines = ["# PEE validation (Fig. 4.1 analog), %d partitions" % len(F), "",
             "Estimated (`sg_plan_info.partition_time`, the PEE on the code generator's pruned work) vs measured "
             "(`sg_profile_partitions`, kernel alone, CUDA events) ns per iteration.", "",
             "* R^2 (linear): %.3f" % r2(est, mea),
             "* R^2 (log-log): %.3f" % r2([math.log(x) for x in est], [math.log(y) for y in mea]),
             "* measured / estimated: median %.2f, min %.2f, max %.2f" % (ratios[len(ratios) // 2], ratios[0],
                                                                          ratios[-1]),
             "", "| config | G | plan | part | nodes | mode | flops/iter | est ns/iter | meas ns/iter | meas/est |",
             "|---|---|---|---|---|---|---|---|---|---|"]
    for f in F:
        kw = ",".join(f"{k}={v}" for k, v in f["kw"].items() if k != "node_partition") or "default"
        if "node_partition" in f["kw"]:
            kw += ",user split"
        lines.append("| %s | %d | %s | %d | %d | %d | %.0f | %.4g | %.4g | %.2f |" % (
            f["config"], f["G"], kw, f["part"], f["nodes"], f["mode"], f["flops"], f["est"], f["meas"],
            f["meas"] / f["est"]))
    print("\n".join(lines[:8]))
    if args.out:
        open(args.out + ".md", "w").write("\n".join(lines) + "\n")
        json.dump(F, open(args.out + ".json", "w"), indent=0)


if __name__ == "__main__":
    main()
