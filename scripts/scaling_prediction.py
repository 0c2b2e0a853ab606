#!/usr/bin/env python
"""Multi-GPU scaling predicted from measured partition times (one B200; the pool has no multi-GPU box).

For each BASELINE multi-GPU config and G = 1, 2, 4, 8 the planner's pipelined plan (replicas = 1,
Algorithm 1 + ILP, chain fission considered -- SURVEY.md 8(e)) and its hybrid replica x pipeline plan
(replicas = -1; the input on one GPU) are built; every partition's kernel is
timed alone at the bench's per-step iteration count (sg_profile_partitions), and the throughput of the
G-GPU pipeline is bounded by ("Tmax ... determines the application throughput"):

  compute:  max over GPUs of the summed partition times on that GPU (Eq. III.4), and
  links:    max over NVSwitch up/down links of the PDG bytes they carry (Eq. III.6-III.7; a duplicated
            stream counted once per destination GPU) / 900 GB/s (NVLink 5 per direction).

It also runs the plan on G virtual GPUs of this device (every partition and ring on one B200) and
reports that time against the summed partition times: the cost of the fragment pipeline itself.

    python scripts/scaling_prediction.py [--out profiles/r02_scaling_prediction]
"""
import argparse
import json
import os
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

N = {"filterbank64": 1 << 22, "fmradio10": 1 << 24, "beamformer12x4": 4096}
IN_ITEMS = {"filterbank64": lambda n: 8 * n, "fmradio10": lambda n: 379 + 5 * n, "beamformer12x4": lambda n: 24576 * n}
LINK_GBS = 900.0


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--out", default=os.path.join(ROOT, "profiles", "r02_scaling_prediction"))
    ap.add_argument("--configs", default=",".join(N))
    args = ap.parse_args()
    import torch
    from paper_conf_cgo_nguyenl16_b200 import sg
    from workloads import apps, inputs
    rows = []
    for name in args.configs.split(","):
        prog = apps.CONFIGS[name]()
        n = N[name]
        x = torch.from_numpy(inputs.make_input("f32", IN_ITEMS[name](n), 7)).cuda()
        base = None
        for G, R in ((1, 1), (2, 1), (4, 1), (8, 1), (2, -1), (4, -1), (8, -1)):
            with sg.plan(prog, G, virtual_gpus=1, replicas=R) as p:
                info = p.info()
                if R == -1 and info["replicas"] == 1:
                    continue                           # the auto model kept the pipeline: row above
                meas = p.profile_partitions(n, 5)
                Rr = info["replicas"]
                Gs = G // Rr
                load = [0.0] * Gs
                for k, g in enumerate(info["partition_gpu"]):
                    load[g] += meas[k] / Rr             # each group runs 1/R of the fragments
                up, down = [0.0] * G, [0.0] * G
                for r in range(Rr):
                    for a, b, nbytes in p.pdg():      # sg_plan_pdg: per (partition pair, stream)
                        ga, gb = info["partition_gpu"][a], info["partition_gpu"][b]
                        if ga != gb:
                            up[r * Gs + ga] += nbytes / Rr
                            down[r * Gs + gb] += nbytes / Rr
                    if r:  # other groups' input / output cross the links of group 0's input / output GPU
                        # (node 0 consumes the graph input, the last node produces the output)
                        gin = info["partition_gpu"][info["node_partition"][0]]
                        gout = info["partition_gpu"][info["node_partition"][-1]]
                        bi, bo = 4.0 * info["in_per_iter"] / Rr, 4.0 * info["out_per_iter"] / Rr
                        up[gin] += bi
                        down[r * Gs + gin] += bi
                        up[r * Gs + gout] += bo
                        down[gout] += bo
                comp = max(load)
                link = max(up + down) / LINK_GBS    # ns per iteration (bytes / (GB/s) = ns)
                if G == 1:
                    base = comp
                # the fragment pipeline on G virtual GPUs of this one device
                y = torch.empty(p.output_items(n), device="cuda")
                p.run(x, n, y)
                torch.cuda.synchronize()
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                e0.record()
                for _ in range(3):
                    p.run(x, n, y)
                e1.record()
                torch.cuda.synchronize()
                virt = e0.elapsed_time(e1) / 3 * 1e6 / n
                row = {"config": name, "G": G, "replicas": Rr, "n_iters": n, "partitions": info["n_partitions"],
                       "chain_fission": info["chain_fission"], "partition_gpu": info["partition_gpu"],
                       "partition_ns": meas, "max_gpu_ns": comp, "link_ns": link,
                       "pred_speedup_compute": base / comp, "pred_speedup": base / max(comp, link),
                       "virtual_run_ns": virt, "sum_partition_ns": sum(meas)}
                rows.append(row)
                print(json.dumps({k: v for k, v in row.items() if k != "partition_ns"}), flush=True)
    json.dump(rows, open(args.out + ".json", "w"), indent=1)
    lines = ["# Multi-GPU scaling predicted from measured partition times (one B200)", "",
             "Per config and G: the planner's pipelined plan (replicas = 1); partition kernels timed alone "
             "(`sg_profile_partitions`, ns per iteration); compute bound = the busiest GPU's summed partition "
             "times; link bound = the busiest NVSwitch link's PDG bytes / 900 GB/s; predicted speedup = "
             "T(1 GPU) / max(compute, link).  `virtual run` = the whole plan run on G virtual GPUs of this one "
             "device (fragment pipeline overhead vs the summed partition times).", "",
             "| config | G | replica groups | partitions | chain | busiest GPU ns/iter | link ns/iter | speedup (compute) | "
             "speedup (compute + links) | x linear | virtual run / sum of partitions |", "|---|---|---|---|---|---|---|---|---|---|---|"]
    for r in rows:
        lines.append("| %s | %d | %d | %d | %s | %.4g | %.4g | %.2f | %.2f | %.2f | %.2f |" % (
            r["config"], r["G"], r["replicas"], r["partitions"], "yes" if r["chain_fission"] else "no", r["max_gpu_ns"],
            r["link_ns"], r["pred_speedup_compute"], r["pred_speedup"], r["pred_speedup"] / r["G"],
            r["virtual_run_ns"] / r["sum_partition_ns"]))
    open(args.out + ".md", "w").write("\n".join(lines) + "\n")
    print("\n".join(lines))


if __name__ == "__main__":
    main()
