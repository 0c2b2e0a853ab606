#!/usr/bin/env python
"""Summarise an `ncu --page source --csv --print-source sass` export: stall samples per
reason, instruction mix, and where in the code the samples fall (address buckets)."""
import csv
import sys
from collections import Counter, defaultdict

path = sys.argv[1]
bucket = int(sys.argv[2]) if len(sys.argv) > 2 else 512
rows = list(csv.reader(open(path)))
hdr_i = next(i for i, r in enumerate(rows) if r and r[0] == "Address")
hdr = rows[hdr_i]
ix = {h: i for i, h in enumerate(hdr)}
stall_cols = [h for h in hdr if h.startswith("stall_") and "Not Issued" not in h]
tot = Counter()
mix = Counter()
byb = defaultdict(Counter)
n = 0
for r in rows[hdr_i + 1:]:
    if len(r) != len(hdr) or not r[0].startswith("0x"):
        continue
    op = r[ix["Source"]].split()[0] if r[ix["Source"]].split() else "?"
    if op.startswith("@"):
        op = r[ix["Source"]].split()[1]
    ex = int(r[ix["Instructions Executed"]] or 0)
    mix[op.split(".")[0]] += ex
    for c in stall_cols:
        v = int(r[ix[c]] or 0)
        tot[c] += v
        byb[n // bucket][c] += v
    byb[n // bucket]["_inst"] += ex
    n += 1
S = sum(tot.values())
print(f"{n} SASS instructions, {S} stall samples")
for c, v in tot.most_common(12):
    print(f"  {c:28s} {v:9d} {100*v/S:5.1f}%")
E = sum(mix.values())
print("instruction mix (executed warp instructions):")
for op, v in mix.most_common(14):
    print(f"  {op:10s} {v:12d} {100*v/E:5.1f}%")
print(f"per {bucket}-instruction bucket: samples, top reasons")
for b in sorted(byb):
    c = byb[b]
    s = sum(v for k, v in c.items() if k != "_inst")
    top = ", ".join(f"{k[6:]} {100*v/max(1,s):.0f}%" for k, v in c.most_common(5) if k != "_inst")
    print(f"  [{b*bucket:6d}) {s:8d} samples  inst {c['_inst']:10d}  {top}")
