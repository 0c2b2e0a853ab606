"""Summarise an ncu source page (--page source --csv --print-source sass) by barrier-delimited region:
samples, top stall reasons, executed warp instructions, FFMA share and excess shared wavefronts.
Usage: ncu -i X.ncu-rep --page source --csv --print-source sass > s.csv; python scripts/sass_regions.py s.csv"""
import csv
import sys
from collections import Counter

rows = list(csv.reader(open(sys.argv[1])))
h = rows[1]
ix = {k: i for i, k in enumerate(h)}
stalls = [k for k in h if k.startswith("stall_") and "Not Issued" not in k]
regions, cur = [], None


def new(addr):
    return {"start": addr, "samples": 0, "inst": 0, "ffma": 0, "lds": 0, "excess": 0, "st": Counter(), "n": 0}


for r in rows[2:]:
    if len(r) < len(h):
        continue
    if cur is None:
        cur = new(r[0])
    src = r[ix["Source"]].strip()
    op = src.split()[0] if src else ""
    if op.startswith("@"):
        op = src.split()[1]
    num = lambda k: float(r[ix[k]] or 0) if r[ix[k]] not in ("-", "") else 0.0
    cur["samples"] += num("Warp Stall Sampling (All Samples)")
    cur["inst"] += num("Instructions Executed")
    cur["n"] += 1
    if op.startswith("FFMA"):
        cur["ffma"] += num("Instructions Executed")
    if op.startswith("LDS"):
        cur["lds"] += num("Instructions Executed")
    cur["excess"] += num("L1 Wavefronts Shared Excessive")
    for s in stalls:
        cur["st"][s] += num(s)
    if op.startswith("BAR"):
        regions.append(cur)
        cur = None
if cur:
    regions.append(cur)
tot = sum(g["samples"] for g in regions) or 1
for k, g in enumerate(regions):
    top = ", ".join(f"{s[6:]} {v / max(1, g['samples']) * 100:.0f}%" for s, v in g["st"].most_common(4))
    print(f"region {k:2d} @{g['start']} sass {g['n']:5d}  samples {g['samples'] / tot * 100:5.1f}%  inst {g['inst']:.3e}"
          f"  ffma {g['ffma'] / max(1, g['inst']) * 100:4.0f}%  lds {g['lds']:.2e}  excess_wf {g['excess']:.2e}  | {top}")
