#!/usr/bin/env python
"""Summarise the ncu captures of one round into profiles/ (run here, on the CPU box).

    python scripts/summarize_ncu.py r01

Reads gpurun_out/<round>/full_<config>.ncu-rep (ncu --set full of the main
partition kernel of `bench.py --config <config>`) and
gpurun_out/<round>/launches_<config>.csv (launch lists), writes
profiles/<round>_summary.md, profiles/<round>_<config>_launches.csv and
profiles/ncu_traffic.json (DRAM bytes per launch, read by bench.py).
"""
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
METRICS = [
    ("gpu__time_duration.sum", "duration"),
    ("dram__bytes_read.sum", "DRAM read"),
    ("dram__bytes_write.sum", "DRAM write"),
    ("gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed", "DRAM % of peak"),
    ("sm__throughput.avg.pct_of_peak_sustained_elapsed", "SM % of peak"),
    ("sm__pipe_fma_cycles_active.avg.pct_of_peak_sustained_active", "FMA pipe active %"),
    ("sm__pipe_alu_cycles_active.avg.pct_of_peak_sustained_active", "ALU pipe active %"),
    ("smsp__issue_active.avg.pct_of_peak_sustained_active", "issue active %"),
    ("sm__warps_active.avg.pct_of_peak_sustained_active", "warps active %"),
    ("launch__registers_per_thread", "registers/thread"),
    ("launch__block_size", "block"),
    ("launch__grid_size", "grid"),
    ("launch__shared_mem_per_block_dynamic", "dyn smem/block"),
    ("l1tex__data_bank_conflicts_pipe_lsu_mem_shared.sum", "smem bank conflicts"),
    ("smsp__sass_thread_inst_executed_op_ffma_pred_on.sum", "FFMA thread-instr"),
]
UNITS = {"Gbyte": 1e9, "Mbyte": 1e6, "Kbyte": 1e3, "byte": 1.0}


def raw(rep):
    """One (metrics, stalls) pair per distinct kernel of the capture (the first launch of each)."""
    out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    h, units = rows[0], rows[1]
    res, seen = [], set()
    for v in rows[2:]:
        if len(v) != len(h):
            continue
        k = v[h.index("Kernel Name")] if "Kernel Name" in h else str(len(res))
        if k in seen:
            continue
        seen.add(k)
        res.append((k,) + one(h, units, v))
    return res


def one(h, units, v):
    d = {h[i]: (v[i], units[i]) for i in range(len(h))}
    stalls = []
    for k, (x, _) in d.items():
        if k.startswith("smsp__pcsamp_warps_issue_stalled_") and not k.endswith("not_issued"):
            try:
                stalls.append((k.replace("smsp__pcsamp_warps_issue_stalled_", ""), float(x.replace(",", ""))))
            except ValueError:
                pass
    tot = sum(x for _, x in stalls) or 1.0
    stalls.sort(key=lambda t: -t[1])
    return d, [(k, x / tot) for k, x in stalls[:6]]


def to_bytes(val, unit):
    return float(val.replace(",", "")) * UNITS.get(unit, 1.0)


def main(rnd):
    src = os.path.join(ROOT, "gpurun_out", rnd)
    os.makedirs(os.path.join(ROOT, "profiles"), exist_ok=True)
    lines = [f"# ncu summary, round {rnd}", "",
             "Main partition kernel of `bench.py --config <name> --steps 2 --warmup 3` captured with",
             "`ncu --set full --clock-control none --import-source on -k regex:sg_part[0-9]+$ -s 3 -c 2` (every",
             "partition kernel of the plan; traffic summed over them per launch of each),"
             "(one launch, cold caches, serialised: use for shares and counters, not as the bench value).", ""]
    tpath = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    traffic = json.load(open(tpath)) if os.path.exists(tpath) else {}
    import glob
    names = sorted(os.path.basename(r)[5:-8] for r in glob.glob(os.path.join(src, "full_*.ncu-rep")))
    for name in names:
        rep = os.path.join(src, f"full_{name}.ncu-rep")
        kernels = raw(rep)
        tot_bytes = 0.0
        for kname, d, stalls in kernels:
            lines.append(f"## {name}: {kname}")
            lines.append("")
            lines.append("| metric | value |")
            lines.append("|---|---|")
            for k, label in METRICS:
                if k in d:
                    lines.append(f"| {label} (`{k}`) | {d[k][0]} {d[k][1]} |")
            lines.append(f"| top stall reasons (pc sampling) | {', '.join(f'{k} {x:.0%}' for k, x in stalls)} |")
            lines.append("")
            try:
                tot_bytes += to_bytes(*d["dram__bytes_read.sum"]) + to_bytes(*d["dram__bytes_write.sum"])
            except Exception:
                pass
        if tot_bytes > 0:
            traffic[name] = {"dram_bytes_per_launch": tot_bytes, "kernels": [k for k, _, _ in kernels],
                             "source": f"profiles/{rnd}_summary.md"}
    for launches in sorted(glob.glob(os.path.join(src, "launches_*.csv"))):
        cfg = os.path.basename(launches)[len("launches_"):-4]
        txt = open(launches).read()
        open(os.path.join(ROOT, "profiles", f"{rnd}_{cfg}_launches.csv"), "w").write(txt)
        rows = [r for r in csv.reader(io.StringIO(txt)) if len(r) > 10 and r[0].isdigit()]
        per = {}
        for r in rows:
            per.setdefault(r[4], []).append(float(r[-1].replace(",", "")))
        lines.append(f"## launch list ({cfg}, `bench.py --config {cfg} --steps 5 --warmup 3`)")
        lines.append("")
        tot = sum(sum(v) for v in per.values()) or 1
        lines.append("| kernel | launches | mean ns | share of GPU time |")
        lines.append("|---|---|---|---|")
        for k, v in sorted(per.items(), key=lambda kv: -sum(kv[1])):
            lines.append(f"| {k} | {len(v)} | {sum(v) / len(v):.0f} | {sum(v) / tot:.1%} |")
        lines.append("")
    open(os.path.join(ROOT, "profiles", f"{rnd}_summary.md"), "w").write("\n".join(lines) + "\n")
    json.dump(traffic, open(tpath, "w"), indent=1)
    print("\n".join(lines))


if __name__ == "__main__":
    main(sys.argv[1] if len(sys.argv) > 1 else "r01")
