import sys, time, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
from workloads import apps, inputs
from paper_conf_cgo_nguyenl16_b200 import sg

def run(prog, n, G, **kw):
    t = time.time()
    x = inputs.make_input("f32", sg.plan(prog, 1, plan_only=1).input_items(n), 5)
    xd = torch.from_numpy(x).cuda()
    with sg.plan(prog, G, **kw) as p:
        t1 = time.time()
        yd = torch.empty(p.output_items(n), device="cuda")
        p.run(xd, n, yd)
        torch.cuda.synchronize()
        print(f"{prog.name} n={n} G={G} {kw}: plan {t1-t:.1f}s run {time.time()-t1:.2f}s parts {p.info()['n_partitions']} launches {p.last_launch_count()}", flush=True)
        return yd.cpu().numpy()

case = sys.argv[1]
fb = apps.filterbank(int(sys.argv[2]) if len(sys.argv) > 2 else 8)
n = int(sys.argv[3]) if len(sys.argv) > 3 else 3000
G = int(sys.argv[4]) if len(sys.argv) > 4 else 2
base = run(fb, n, 1)
if case == "chain":
    y = run(fb, n, G, virtual_gpus=1, chain_groups=G, partitioner="chain", iters_per_fragment=max(1, n // 7))
elif case == "chain1":
    y = run(fb, n, 1, chain_groups=G, partitioner="single")
elif case == "planner":
    y = run(fb, n, G, virtual_gpus=1, replicas=1)
elif case == "perfilter":
    y = run(fb, n, G, virtual_gpus=1, partitioner="per_filter", iters_per_fragment=max(1, n // 5))
print(case, "bit-identical" if y.tobytes() == base.tobytes() else "DIFFERENT", flush=True)
