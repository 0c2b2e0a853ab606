#!/usr/bin/env python
"""Benchmark of the steady-state stream-graph path (BASELINE.json metric).

    python bench.py [--gpus N] [--steps K] [--warmup W] [--config NAME] [--impl sg|reference]

One step = one sg_run() over the whole workload (replayed as a CUDA graph) (all of SURVEY.md 8(a)'s timed
rows: tile loads, filter execution, stores; plus boundary streams when the plan
has several partitions/GPUs).  Default workload: the largest graph of BASELINE.json
(configs[4], FilterBank 64 branches fp32, the north star's "largest graph"), 2^20
iterations on one GPU.  Inputs resident in HBM; L2 flushed (256 MiB write + read-back
with our sg_flush_l2 kernels) before every timed step, outside the per-step CUDA-event
window.  Under torchrun (N > 1) the default is the paper's pipelined mapping
(--mode pipeline): every rank builds the same plan for N GPUs (Algorithm 1 + ILP; for
FilterBank the chain-fission groups) and runs its partitions with NCCL
boundary streams (sg_run_rank), 2^24 iterations per step so the fragment pipeline
fills; value = iterations / max-over-ranks time ("strong").  --mode replicas runs N
independent replicas instead ("weak").  --config fft64 also reports BASELINE's 4096
iterations (CUDA-graph replay) next to the 2^20 roofline run.

--impl reference times the oracle (the plain sequential CPU interpreter in
oracle/, as it stands) on the host cores, on a bounded sample of the workload.
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

METRIC = "steady-state iters/s (output items/s) at 1/2/4/8 B200; % of roofline"

# workload table: iterations per step, roofline class, algorithmic bytes / ops per iteration
WORKLOADS = {
    "bitonic32": dict(n=1 << 20, bound="hbm", desc="BitonicSort 32-key int32, 1M iterations"),
    "fft64": dict(n=1 << 20, bound="hbm", desc="StreamIt FFT2 N=64 fp32 (2 x 64-pt complex FFT per iteration)"),
    "fmradio10": dict(n=1 << 24, bound="alu", desc="FMRadio + 10-band equalizer fp32"),
    "beamformer12x4": dict(n=4096, bound="alu", desc="BeamFormer 12 channels x 4 beams fp32, 1024-sample frames"),
    "filterbank64": dict(n=1 << 20, bound="alu", desc="FilterBank 64 branches fp32 (M=8, L=32)"),
    # second workloads of the paper's suite, not BASELINE configs
    "bitonicrec32": dict(n=1 << 20, bound="hbm", desc="recursive BitonicSort 32-key int32, 1M iterations"),
    "dct16": dict(n=1 << 18, bound="hbm", desc="2-D DCT-II of 16x16 fp32 blocks (row then column FIR DCTs)"),
    "matmul16": dict(n=1 << 18, bound="hbm", desc="C = A B of streamed 16x16 fp32 matrices (MULTIPLY, ADD)"),
    "matmul3_16": dict(n=1 << 18, bound="hbm", desc="MatMul3: blocked C = sum_d A_d B_d, 16x16 fp32, 4 K-blocks"),
    # feedback loops: the comb loop is a sequential (wavefront) partition between two FIRs
    "echo64": dict(n=1 << 22, bound="alu", desc="echo: FIR -> feedback loop y = x + 0.5 y[n-64] -> decimating FIR, fp32"),
    "des16": dict(n=1 << 22, bound="int", desc="DES (16 rounds) on a bit-per-item int32 stream, one 64-bit block / iteration"),
}


def measured_peaks():
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as f:
            return json.load(f), "measured"
    except Exception:
        return {"hbm_gbs": 6650.0, "sm_max_mhz": 1965.0}, "fallback"


class ClockSampler:
    """nvidia-smi clocks + throttle reasons, sampled in the background during the timed region."""

    FIELDS = ["clocks.sm", "clocks.max.sm", "clocks_event_reasons.active",
              "clocks_event_reasons.hw_slowdown", "clocks_event_reasons.hw_thermal_slowdown",
              "clocks_event_reasons.sw_thermal_slowdown", "clocks_event_reasons.sw_power_cap"]

    def __init__(self, gpu_index: int):
        self.idx = gpu_index
        self.rows = []
        self.proc = None
        self.t = None

    def start(self):
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", f"--id={self.idx}", "--query-gpu=" + ",".join(self.FIELDS),
                 "--format=csv,noheader,nounits", "-lms", "50"],
                stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
        except Exception:
            self.proc = None
            return
        self.t = threading.Thread(target=self._read, daemon=True)
        self.t.start()

    def _read(self):
        for line in self.proc.stdout:
            parts = [p.strip() for p in line.split(",")]
            if len(parts) == len(self.FIELDS):
                self.rows.append(parts)

    def stop(self):
        if self.proc is None:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["nvidia-smi unavailable"], "samples": 0}
        time.sleep(0.12)
        self.proc.terminate()
        try:
            self.proc.wait(timeout=2)
        except Exception:
            self.proc.kill()
        if self.t:
            self.t.join(timeout=2)
        sm = [float(r[0]) for r in self.rows if r[0].replace(".", "").isdigit()]
        mx = [float(r[1]) for r in self.rows if r[1].replace(".", "").isdigit()]
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = set()
        for r in self.rows:
            for k, nm in enumerate(names):
                if r[3 + k].lower().startswith("active"):
                    reasons.add(nm)
        return {"sm_mhz": statistics.median(sm) if sm else None, "sm_max_mhz": max(mx) if mx else None,
                "reasons": sorted(reasons), "samples": len(self.rows)}


def cpu_baseline(prog, name, target_s=10.0):
    """The oracle as it stands, on a bounded sample of the workload, one host core."""
    from oracle import oracle as O
    from workloads import inputs
    n_total = WORKLOADS[name]["n"]
    n0 = 16 if name == "beamformer12x4" else 4096
    x = inputs.make_input(prog.dtype, O.in_items(prog, n0), inputs.SEEDS[name])
    t = time.perf_counter()
    O.run(prog, x, n0)
    rate = n0 / max(1e-6, time.perf_counter() - t)
    n = int(min(n_total, max(n0, rate * target_s)))
    # input long enough for n iterations without bisecting in_items(n) over whole-program runs:
    # in_items(k * n0) <= k * in_items(n0) (per-iteration input plus one peek halo); extra input is unread
    reps = -(-n // n0)
    x = inputs.make_input(prog.dtype, reps * O.in_items(prog, n0), inputs.SEEDS[name])
    t = time.perf_counter()
    O.run(prog, x, n)
    dt = time.perf_counter() - t
    out = {"value": n / dt, "unit": "iters/s", "cores": 1, "kind": "oracle",
           "sample": f"first {n} of {n_total} iterations of {name} (seeded input), sequential C interpreter, "
                     f"{dt:.1f} s, gcc -O2 -ffp-contract=off"}
    # all host cores: the same interpreter on independent chunks of iterations, one thread per core
    # (ctypes releases the GIL during the C call); each chunk restarts at a stream start, which changes
    # peek-halo values but not the work
    cores = min(os.cpu_count() or 1, 64)
    if cores > 1 and not os.environ.get("SG_ORACLE_1CORE"):
        from concurrent.futures import ThreadPoolExecutor
        out_per_iter = max(1, len(O.run(prog, x, 1)))
        nc = max(n0, min(int(rate * target_s / 2), int(1e9 / (cores * 4 * out_per_iter))))  # <= 1 GB of outputs
        xc = inputs.make_input(prog.dtype, -(-nc // n0) * O.in_items(prog, n0), inputs.SEEDS[name])
        t = time.perf_counter()
        with ThreadPoolExecutor(cores) as ex:
            list(ex.map(lambda _: O.run(prog, xc, nc), range(cores)))
        dtc = time.perf_counter() - t
        out.update({"value": cores * nc / dtc, "cores": cores, "value_1core": n / dt,
                    "sample": out["sample"] + f"; all cores: {cores} threads x {nc} iterations each, {dtc:.1f} s"})
    return out


def run_reference(args):
    rank = int(os.environ.get("RANK", "0"))
    if rank != 0:
        return 0
    from workloads import apps
    name = args.config
    prog = {**apps.CONFIGS, **apps.EXTRA, **apps.FEEDBACK}[name]()
    vals = []
    cb = None
    for _ in range(max(1, args.warmup)):
        pass  # the oracle has no warm state worth excluding beyond the first call below
    for k in range(args.steps if args.steps <= 3 else 3):
        cb = cpu_baseline(prog, name, target_s=5.0)
        vals.append(cb["value"])
    v = statistics.median(vals)
    cb["value"] = v
    line = {"impl": "reference", "metric": METRIC, "value": v, "unit": "iters/s", "n_gpus": args.gpus,
            "steps": len(vals), "warmup": args.warmup,
            # the time one step of the full workload would take at the sampled rate (each step timed a sample)
            "ms_per_step": WORKLOADS[name]["n"] / v * 1e3 if v > 0 else None, "higher_is_better": True,
            "scaling": "weak", "vs_baseline": None, "dtype": "i32" if prog.dtype == "i32" else "f32",
            "data": "synthetic", "config": {"workload": name, "desc": WORKLOADS[name]["desc"],
                                             "iters": WORKLOADS[name]["n"], "sample": cb["sample"]},
            "cpu_baseline": cb, "e2e": {"value": v, "unit": "iters/s", "h2d_bytes_per_step": 0,
                                        "d2h_bytes_per_step": 0}}
    print(json.dumps(line))
    return 0


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=3000)
    ap.add_argument("--warmup", type=int, default=20)
    ap.add_argument("--config", default="filterbank64", choices=list(WORKLOADS))
    ap.add_argument("--impl", default="sg", choices=["sg", "reference"])
    ap.add_argument("--iters", type=int, default=0, help="override iterations per step")
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--no-flush", action="store_true")
    ap.add_argument("--eager", action="store_true", help="launch sg_run every step instead of replaying a CUDA graph")
    ap.add_argument("--tile", type=int, default=0, help="plan option tile_iters (0: chosen by the code generator)")
    ap.add_argument("--threads", type=int, default=0, help="plan option threads per CTA (0: chosen)")
    ap.add_argument("--replicas", type=int, default=1,
                    help="--mode pipeline: replica groups (hybrid replica x pipeline plan); -1 = chosen by the cost model")
    ap.add_argument("--cuts", default="",
                    help="comma-separated node ids: user partitions [0, c1), [c1, c2), ... on one GPU (A/B of splits)")
    ap.add_argument("--node-partition", default="",
                    help="comma-separated partition id per node: user partitions on one GPU (A/B of non-contiguous "
                         "splits)")
    ap.add_argument("--chain", type=int, default=0,
                    help="1 GPU: plan option chain_groups (chain fission of the largest eligible split-join, one "
                         "partition); 0 = as planned")
    ap.add_argument("--codegen", default="auto", choices=["auto", "register", "staged", "general"],
                    help="plan option codegen_mode (auto: chosen by the code generator)")
    ap.add_argument("--force-pipeline", action="store_true",
                    help="run the one-process-per-GPU pipelined path (sg_run_rank, NCCL) even on one GPU (a check "
                         "of the multi-GPU bench path on a one-GPU box)")
    ap.add_argument("--mode", default="pipeline", choices=["replicas", "pipeline"],
                    help="N>1: the paper's pipelined partition mapping (default), one process per GPU, NCCL "
                         "boundary streams; or independent replicas")
    args = ap.parse_args()
    if args.warmup < 3:
        args.warmup = 3
    if args.impl == "reference":
        return run_reference(args)

    import torch
    import torch.distributed as dist
    from paper_conf_cgo_nguyenl16_b200 import sg
    from workloads import apps, inputs

    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    if args.force_pipeline and world == 1:
        os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
        os.environ.setdefault("MASTER_PORT", "29531")
        os.environ.setdefault("RANK", "0")
        os.environ.setdefault("WORLD_SIZE", "1")
    if world > 1 or args.force_pipeline:
        dist.init_process_group("nccl", device_id=torch.device("cuda", local))
    torch.cuda.set_device(local)
    name = args.config
    W = WORKLOADS[name]
    pipeline = args.mode == "pipeline" and (world > 1 or args.force_pipeline)
    # pipelined runs need many fragments per GPU (fill / drain F / (F + G - 1))
    n = args.iters or (max(W["n"], 1 << 24) if pipeline and W["bound"] == "alu" and name != "beamformer12x4"
                       else W["n"])
    prog = {**apps.CONFIGS, **apps.EXTRA, **apps.FEEDBACK}[name]()
    if pipeline:
        from paper_conf_cgo_nguyenl16_b200.dist import pipeline_plan
        plan = pipeline_plan(prog, replicas=args.replicas)
    else:
        kw = {}
        if args.tile:
            kw["tile_iters"] = args.tile
        if args.threads:
            kw["threads"] = args.threads
        if args.codegen != "auto":
            kw["codegen_mode"] = args.codegen
        if args.chain:
            kw["chain_groups"] = args.chain
            kw["partitioner"] = "single"
        if args.cuts:
            cuts = [int(c) for c in args.cuts.split(",")]
            with sg.plan(prog, 1, plan_only=1) as p0:
                nn = p0.info()["n_nodes"]
            kw["node_partition"] = [sum(1 for c in cuts if c <= v) for v in range(nn)]
        if args.node_partition:
            kw["node_partition"] = [int(c) for c in args.node_partition.split(",")]
        plan = sg.plan(prog, 1, devices=[local], **kw)
    info = plan.info()
    nin, nout = plan.input_items(n), plan.output_items(n)
    dt = torch.int32 if prog.dtype == "i32" else torch.float32
    x_host = torch.from_numpy(inputs.make_input(prog.dtype, nin, inputs.SEEDS[name] + (0 if pipeline else rank)))
    x = x_host.to(f"cuda:{local}")
    y = torch.empty(nout, dtype=dt, device=f"cuda:{local}")
    flush = torch.empty(256 << 20, dtype=torch.uint8, device=f"cuda:{local}")
    stream = torch.cuda.current_stream()

    run_step = (lambda: plan.run_rank(x, n, y, stream)) if pipeline else (lambda: plan.run(x, n, y, stream))
    for _ in range(args.warmup):
        run_step()
    launches_per_step = plan.last_launch_count()
    torch.cuda.synchronize()
    # CUDA graph of one sg_run (the C ABI call enqueues only kernels and events on the
    # capturing stream); replaying it removes host launch gaps from the timed window.
    graph = None
    if not args.eager and not pipeline:
        try:
            gs = torch.cuda.Stream()
            graph = torch.cuda.CUDAGraph()
            with torch.cuda.graph(graph, stream=gs):
                plan.run(x, n, y, torch.cuda.current_stream())
            torch.cuda.synchronize()
            for _ in range(args.warmup):
                graph.replay()
            torch.cuda.synchronize()
        except Exception as exc:  # capture not possible (e.g. multi-GPU plan): eager launches
            print(f"[bench] CUDA graph capture failed ({exc}); eager launches", file=sys.stderr)
            graph = None
            torch.cuda.synchronize()

    def step():
        if graph is not None:
            graph.replay()
        else:
            run_step()

    ev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)) for _ in range(args.steps)]
    sampler = ClockSampler(local)
    if dist.is_initialized():
        dist.barrier()
    torch.cuda.synchronize()
    sampler.start()
    time.sleep(0.15)
    wall0 = time.perf_counter()
    for k in range(args.steps):
        if not args.no_flush:
            sg.flush_l2(flush, stream.cuda_stream)
        ev[k][0].record(stream)
        step()
        ev[k][1].record(stream)
    torch.cuda.synchronize()
    wall = time.perf_counter() - wall0
    if dist.is_initialized():
        dist.barrier()
    clocks = sampler.stop()
    step_ms = [a.elapsed_time(b) for a, b in ev]
    total_ms = sum(step_ms)
    if world > 1:
        t = torch.tensor([total_ms], dtype=torch.float64, device=f"cuda:{local}")
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
        total_ms = float(t.item())
    ms_per_step = total_ms / args.steps
    value = (1 if pipeline else world) * n * args.steps / (total_ms / 1e3)

    # roofline of the dominant kernel (single partition: one launch per step)
    peaks, peak_src = measured_peaks()
    # kernel duration: CUDA events around the launch on its stream (one kernel per step here)
    # one partition => every launch of the step is this partition's kernel (main + stream-start variant)
    # one GPU, several partitions: the step's kernels run back to back on one device; the roofline is
    # then that of the whole step (every launch is one of the plan's partition kernels)
    # (feedback loops excepted: their partition is a serial chain, bounded by latency, not by a roof)
    serial = 4 in info["partition_mode"]
    kern_ms = statistics.median(step_ms) if (info["n_partitions"] == 1 or (world == 1 and not pipeline and not serial)) else None
    ki_bytes = (info["in_per_iter"] + info["out_per_iter"]) * 4 * n
    roof = None
    if W["bound"] == "hbm":
        if kern_ms:
            ach = ki_bytes / (kern_ms / 1e3) / 1e9
            roof = {"bound": "hbm", "achieved": ach, "peak": peaks["hbm_gbs"], "unit": "GB/s",
                    "frac": ach / peaks["hbm_gbs"], "traffic": None,
                    "algorithmic_bytes_per_launch": ki_bytes, "peak_source": peak_src + " copy bandwidth"}
    elif W["bound"] == "int":
        # DES works on one bit per item: its algorithmic ops are bit operations, and the ALU's peak in
        # bit operations is 32 per int32 lane op (the bitsliced kernel packs 32 iterations per word)
        ops = info["intops_per_iter"]
        if kern_ms:
            ach = ops * n / (kern_ms / 1e3) / 1e12
            pk = 148 * 64 * 32 * peaks.get("sm_max_mhz", 1965.0) * 1e6 / 1e12
            roof = {"bound": "alu", "achieved": ach, "peak": pk, "unit": "Tbitops/s", "frac": ach / pk,
                    "traffic": None, "algorithmic_ops_per_launch": ops * n, "ops_per_iter": ops,
                    "ops_counting": "as written, in bit operations: one per XORed bit (key XOR included), one per "
                                    "S-box lookup, one per bit unpacked / packed",
                    "peak_source": "derived: 148 SMs x 64 int32 lanes/clk (alu pipe: LOP3/SHF) x 32 bits x sm_max_mhz"}
    else:
        fl_written = _flops_per_iter(prog, info["reps"])
        fl = min(fl_written, info["flops_per_iter_pruned"]) if info["flops_per_iter_pruned"] > 0 else fl_written
        if kern_ms:
            ach = fl * n / (kern_ms / 1e3) / 1e12
            pk = 148 * 128 * 2 * peaks.get("sm_max_mhz", 1965.0) * 1e6 / 1e12
            roof = {"bound": "alu", "achieved": ach, "peak": pk, "unit": "TFLOP/s", "frac": ach / pk,
                    "traffic": None, "algorithmic_flops_per_launch": fl * n,
                    "flops_per_iter": fl, "flops_per_iter_as_written": fl_written,
                    "flops_counting": "as written" if fl == fl_written else
                    "pruned (dead firings and zero taps eliminated by the code generator)",
                    "peak_source": "derived: 148 SMs x 128 FP32 lanes x 2 x sm_max_mhz (FFMA)"}
    if roof is not None:
        roof["scope"] = ("the partition kernel (one launch per step, plus the stream-start variant beside it)"
                         if info["n_partitions"] == 1 else
                         f"the whole step: {info['n_partitions']} partition kernels back to back on one GPU")
    prof = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    # (per-launch DRAM bytes of one kernel; a multi-partition step launches each kernel once per fragment,
    # so only one-partition steps carry it -- the profiles/ summary lists every kernel's own)
    if roof is not None and os.path.exists(prof) and info["n_partitions"] == 1:
        try:
            tr = json.load(open(prof)).get(name)
            if tr:
                roof["traffic"] = tr["dram_bytes_per_launch"]
        except Exception:
            pass

    # end to end through the public C ABI with HOST buffers (pinned), copies inside the timed region
    e2e = None
    if pipeline:
        # one process per GPU: the input rank copies the step's input in from pinned host memory, the
        # output rank copies the output back; wall clock between barriers, max over ranks
        xh = x_host.pin_memory()
        yh = torch.empty(nout, dtype=dt).pin_memory()
        is_in, is_out = local == info["input_device"], local == info["output_device"]
        k2 = max(3, min(10, args.steps))
        torch.cuda.synchronize()
        dist.barrier()
        t0 = time.perf_counter()
        for _ in range(k2):
            if is_in:
                x.copy_(xh, non_blocking=True)
            plan.run_rank(x, n, y, stream)
            if is_out:
                yh.copy_(y, non_blocking=True)
            torch.cuda.synchronize()
        dist.barrier()
        e2e_s = (time.perf_counter() - t0) / k2
        from paper_conf_cgo_nguyenl16_b200.dist import max_over_ranks
        e2e_s = max_over_ranks(e2e_s, device=f"cuda:{local}")
        e2e = {"value": n / e2e_s, "unit": "iters/s", "h2d_bytes_per_step": nin * 4, "d2h_bytes_per_step": nout * 4,
               "steps": k2, "timing": "host wall clock between barriers around H2D (input rank) + sg_run_rank + "
                                      "D2H (output rank), max over ranks"}
    else:
        xh = x_host.pin_memory()
        yh = torch.empty(nout, dtype=dt).pin_memory()
        xnp, ynp = xh.numpy(), yh.numpy()
        plan.run_host(xnp, n, ynp)
        k2 = max(3, min(20, args.steps))
        t0 = time.perf_counter()
        for _ in range(k2):
            plan.run_host(xnp, n, ynp)
        e2e_s = (time.perf_counter() - t0) / k2
        e2e = {"value": world * n / e2e_s, "unit": "iters/s", "h2d_bytes_per_step": nin * 4,
               "d2h_bytes_per_step": nout * 4, "steps": k2, "timing": "host wall clock around sg_run_host"}

    # FFT: BASELINE.json configs[0] is 4096 iterations (8 MiB of traffic, ~1 us at the roof, L2-resident):
    # a step is one sg_run of 4096 iterations; one replay of a graph of one sg_run is bound by the host's
    # graph-launch rate, so the graph holds GPS back-to-back steps (each its own sg_run on its own output)
    # and is replayed REPS times: device time per step.  The one-run-per-replay rate is kept beside it.
    at_config = None
    if name == "fft64" and not pipeline and world == 1:
        n4, GPS, REPS = 4096, 64, 32
        y4 = torch.empty(plan.output_items(n4), dtype=dt, device=f"cuda:{local}")

        def graph_of(k):
            g = torch.cuda.CUDAGraph()
            with torch.cuda.graph(g, stream=torch.cuda.Stream()):
                for _ in range(k):
                    plan.run(x, n4, y4, torch.cuda.current_stream())
            return g

        def time_graph(g, reps):
            for _ in range(5):
                g.replay()
            torch.cuda.synchronize()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(stream)
            for _ in range(reps):
                g.replay()
            e1.record(stream)
            torch.cuda.synchronize()
            return e0.elapsed_time(e1) / reps

        ms4 = time_graph(graph_of(GPS), REPS) / GPS
        ms1 = time_graph(graph_of(1), 1000)
        at_config = {"iters_per_step": n4, "value": n4 / (ms4 / 1e3), "unit": "iters/s", "ms_per_step": ms4,
                     "steps": GPS * REPS,
                     "note": f"BASELINE.json configs[0] size: a CUDA graph of {GPS} back-to-back sg_run steps replayed "
                             f"{REPS} times, L2-resident (8 MiB), not flushed",
                     "one_step_per_graph_replay": {"value": n4 / (ms1 / 1e3), "ms_per_step": ms1,
                                                   "note": "1000 replays of a graph of one sg_run (host launch rate)"}}

    cb = None
    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        cb = cpu_baseline(prog, name)

    if rank == 0:
        line = {
            "metric": METRIC, "value": value, "unit": "iters/s", "n_gpus": world, "steps": args.steps,
            "warmup": args.warmup, "ms_per_step": ms_per_step, "higher_is_better": True,
            "scaling": "strong" if pipeline else "weak",
            "vs_baseline": None, "dtype": "i32" if prog.dtype == "i32" else "f32", "data": "synthetic",
            "config": {"workload": name, "desc": W["desc"], "iters_per_step": n,
                       "items_per_s_out": value * info["out_per_iter"],
                       "l2": "flushed before every step (256 MiB sg_flush_l2: write + read back), outside the event window"
                       if not args.no_flush else "not flushed",
                       "chain_fission": info["chain_fission"], "partition_gpu": info["partition_gpu"],
                       "parallelism": (f"pipeline over {world} GPUs (ILP mapping, NCCL boundary streams)" if pipeline
                                       else f"replicas x{world}" if world > 1
                                       else f"1 GPU, {info['n_partitions']} partition(s)"),
                       "partitions": info["n_partitions"], "partition_mode": info["partition_mode"],
                       "launch": "CUDA graph replay of one sg_run" if graph is not None else "eager sg_run",
                       "wall_s": wall},
            "roofline": roof, "cpu_baseline": cb, "e2e": e2e,
            **({"at_config_size": at_config} if at_config else {}),
            "gpu_launches": args.steps * (launches_per_step + (0 if args.no_flush else 2)),
            "clocks": clocks,
        }
        print(json.dumps(line))
    plan.close()
    if dist.is_initialized():
        dist.destroy_process_group()
    return 0


def _flops_per_iter(prog, reps):
    """Algorithmic fp32 flops per iteration as written (FMA = 2): program text x repetition vector."""
    from workloads.spec import FeedbackLoop, Filter, Pipeline
    k = [0]
    tot = [0]

    def walk(s):
        if isinstance(s, FeedbackLoop):   # one N_LOOP node in the product's flat graph (its work not counted)
            k[0] += 1
            return
        if isinstance(s, Filter):
            rep = reps[k[0]]
            k[0] += 1
            iv = s.ints
            per = {"FIR": 2 * iv[0] if iv else 0, "COMBINE_DFT": 10 * (iv[0] // 2) if iv else 0, "FM_DEMOD": 1,
                   "SUBTRACT": 1, "AMPLIFY": 1, "ADD": iv[0] if iv else 0,
                   "BEAM_FIR": 8 * iv[0] * (iv[2] // iv[1]) if len(iv) >= 3 else 0,
                   "BEAMFORM": 8 * iv[0] if iv else 0, "MAGNITUDE": 3}.get(s.kind, 0)
            tot[0] += per * rep
        elif isinstance(s, Pipeline):
            for c in s.children:
                walk(c)
        else:
            k[0] += 1
            for b in s.branches:
                walk(b)
            k[0] += 1

    walk(prog.top)
    return tot[0]


if __name__ == "__main__":
    sys.exit(main())
