"""Summarise bench.py JSON lines (gpurun_out/<tag>/bench_*.json) as a markdown table."""
import glob
import json
import sys

tag = sys.argv[1]
rows = []
for fn in sorted(glob.glob(f"gpurun_out/{tag}/bench_*.json")):
    try:
        d = json.loads(open(fn).read().strip().splitlines()[-1])
    except Exception:
        continue
    r = d.get("roofline") or {}
    c = d.get("config", {})
    rows.append((c.get("workload", fn), d["value"], d["ms_per_step"], r.get("bound"), r.get("achieved"), r.get("peak"),
                 r.get("unit"), r.get("frac"),
                 "%s (%s cores)" % (("%.3g" % (d.get("cpu_baseline") or {}).get("value", float("nan"))),
                                    (d.get("cpu_baseline") or {}).get("cores")) if d.get("cpu_baseline") else None,
                 (d.get("e2e") or {}).get("value"),
                 (d.get("clocks") or {}).get("sm_mhz")))
print("| workload | iters/s | ms/step | bound | achieved | peak | unit | frac | oracle iters/s (host cores) | e2e iters/s | SM MHz |")
print("|---|---|---|---|---|---|---|---|---|---|---|")
for w in rows:
    f = lambda x, p=3: ("%.*g" % (p, x)) if isinstance(x, (int, float)) else str(x)
    print(f"| {w[0]} | {f(w[1], 4)} | {f(w[2], 4)} | {w[3]} | {f(w[4], 4)} | {f(w[5], 4)} | {w[6]} | {f(w[7], 3)} | "
          f"{f(w[8], 3)} | {f(w[9], 3)} | {f(w[10], 4)} |")
