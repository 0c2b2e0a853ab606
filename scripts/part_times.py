"""Per-partition kernel times (sg_profile_partitions, each partition alone) next to the PEE's refined
estimate, for a config's default plan on one GPU.  Usage: python scripts/part_times.py <config> [n_iters]"""
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
from paper_conf_cgo_nguyenl16_b200 import sg  # noqa: E402
from workloads import apps  # noqa: E402

name = sys.argv[1]
n = int(sys.argv[2]) if len(sys.argv) > 2 else 4096
prog = {**apps.CONFIGS, **apps.EXTRA}[name]()
with sg.plan(prog, 1) as p:
    info = p.info()
    meas = p.profile_partitions(n)
    rows = []
    for k in range(info["n_partitions"]):
        f = p.pee_features(k)
        rows.append({"part": k, "est_ns": info["partition_time"][k], "meas_ns": meas[k], "flops": f["flops"],
                     "par_eff": f["par_eff"], "tile": f["tile"], "threads": f["threads"],
                     "tflops": f["flops"] / meas[k] * 1e-3 if meas[k] > 0 else None})
    print(json.dumps({"config": name, "env": {k: v for k, v in os.environ.items() if k.startswith("SG_")},
                      "parts": rows}))
