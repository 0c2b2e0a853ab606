"""Thin ctypes binding of libsg.so (include/sg.h).  Argument marshalling only:
every step of the stream-graph path (rates, planning, code generation, kernels,
transfers) runs in the native library.  There is no CPU fallback: sg_run on a
machine without a CUDA device fails with SG_E_CUDA.

    from paper_conf_cgo_nguyenl16_b200 import sg
    with sg.plan(program, n_gpus=1) as p:          # program: workloads.spec.Program or sg.Graph
        p.run(x_cuda, n_iters, y_cuda)             # device tensors, current torch stream
"""
from __future__ import annotations

import ctypes
import os
from typing import Optional, Sequence

_HERE = os.path.dirname(os.path.abspath(__file__))
_LIB_PATH = os.path.join(_HERE, "libsg.so")
_lib = None

SG_OK, SG_E_ARG, SG_E_STRUCTURE, SG_E_RATE, SG_E_UNSUPPORTED = 0, -1, -2, -3, -4
SG_E_NOMEM, SG_E_CUDA, SG_E_COMM, SG_E_PLAN, SG_E_SIZE = -5, -6, -7, -8, -9
SG_F32, SG_I32 = 0, 1
SG_PART_ALGORITHM1, SG_PART_SINGLE, SG_PART_PER_FILTER, SG_PART_USER, SG_PART_CHAIN = 0, 1, 2, 3, 4

KINDS = {"IDENTITY": 0, "FIR": 1, "DELAY": 2, "DECIMATE": 3, "EXPAND": 4, "COMPARE_EXCHANGE": 5,
         "FFT_REORDER": 6, "COMBINE_DFT": 7, "FM_DEMOD": 8, "SUBTRACT": 9, "AMPLIFY": 10, "ADD": 11,
         "BEAM_FIR": 12, "BEAMFORM": 13, "MAGNITUDE": 14,
         "MULTIPLY": 15, "PERMUTE": 16, "XOR": 17, "XOR_CONST": 18, "SBOX": 19,
         "INTO_BITS": 20, "BITS_TO_INT": 21}

EXPORTS = ["sg_graph_create", "sg_graph_destroy", "sg_add_filter", "sg_add_splitjoin", "sg_add_feedbackloop",
           "sg_branch_begin",
           "sg_branch_end", "sg_plan_opts_default", "sg_plan", "sg_input_items", "sg_output_items",
           "sg_plan_info", "sg_plan_source", "sg_run", "sg_run_host", "sg_last_launch_count",
           "sg_plan_destroy", "sg_last_error", "sg_version", "sg_flush_l2", "sg_topology_links",
           "sg_topology_dtlist", "sg_map_ilp", "sg_paper_model", "sg_plan_pdg", "sg_comm_unique_id", "sg_comm_init",
           "sg_run_rank", "sg_rank_schedule", "sg_profile_partitions", "sg_pee_features"]
SG_OP_LAUNCH, SG_OP_SEND, SG_OP_RECV = 0, 1, 2


class SgError(RuntimeError):
    def __init__(self, code: int, msg: str):
        super().__init__(f"[sg status {code}] {msg}")
        self.code = code


class FilterDesc(ctypes.Structure):
    _fields_ = [("kind", ctypes.c_int), ("n_i", ctypes.c_int32), ("p_i", ctypes.POINTER(ctypes.c_int32)),
                ("n_f", ctypes.c_int32), ("p_f", ctypes.POINTER(ctypes.c_float))]


class PlanOpts(ctypes.Structure):
    _fields_ = [("partitioner", ctypes.c_int32), ("node_partition", ctypes.POINTER(ctypes.c_int32)),
                ("n_node_partition", ctypes.c_int32), ("tile_iters", ctypes.c_int32), ("threads", ctypes.c_int32),
                ("iters_per_fragment", ctypes.c_int64), ("transport", ctypes.c_int32),
                ("virtual_gpus", ctypes.c_int32), ("devices", ctypes.POINTER(ctypes.c_int32)),
                ("ilp_time_limit_ms", ctypes.c_int32), ("codegen_mode", ctypes.c_int32),
                ("link_gbps", ctypes.c_double), ("link_latency_us", ctypes.c_double), ("verbose", ctypes.c_int32),
                ("plan_only", ctypes.c_int32), ("replicas", ctypes.c_int32), ("chain_groups", ctypes.c_int32)]


class RankOp(ctypes.Structure):
    _fields_ = [("op", ctypes.c_int32), ("part", ctypes.c_int32), ("edge", ctypes.c_int32), ("peer", ctypes.c_int32),
                ("fragment", ctypes.c_int64), ("k_begin", ctypes.c_int64), ("k_end", ctypes.c_int64),
                ("items", ctypes.c_int64)]


class PlanInfo(ctypes.Structure):
    _fields_ = [("n_nodes", ctypes.c_int32), ("n_edges", ctypes.c_int32), ("n_partitions", ctypes.c_int32),
                ("n_gpus", ctypes.c_int32), ("in_per_iter", ctypes.c_int64), ("out_per_iter", ctypes.c_int64),
                ("reps", ctypes.POINTER(ctypes.c_int64)), ("init_firings", ctypes.POINTER(ctypes.c_int64)),
                ("node_type", ctypes.POINTER(ctypes.c_int32)), ("node_kind", ctypes.POINTER(ctypes.c_int32)),
                ("node_partition", ctypes.POINTER(ctypes.c_int32)), ("partition_gpu", ctypes.POINTER(ctypes.c_int32)),
                ("partition_time", ctypes.POINTER(ctypes.c_double)),
                ("partition_mode", ctypes.POINTER(ctypes.c_int32)), ("est_tmax", ctypes.c_double),
                ("input_device", ctypes.c_int32), ("output_device", ctypes.c_int32),
                ("iters_per_fragment", ctypes.c_int64), ("ilp_optimal", ctypes.c_int32),
                ("flops_per_iter_written", ctypes.c_double), ("flops_per_iter_pruned", ctypes.c_double),
                ("intops_per_iter", ctypes.c_int64), ("replicas", ctypes.c_int32), ("chain_fission", ctypes.c_int32)]


def lib():
    """Load libsg.so (building it in-tree with nvcc if it is not there yet)."""
    global _lib
    if _lib is not None:
        return _lib
    if not os.path.exists(_LIB_PATH):
        from . import build as _b
        _b.build()
    L = ctypes.CDLL(_LIB_PATH)
    vp, i32, i64 = ctypes.c_void_p, ctypes.c_int32, ctypes.c_int64
    sig = {
        "sg_graph_create": ([ctypes.c_int, ctypes.POINTER(vp)], ctypes.c_int),
        "sg_graph_destroy": ([vp], None),
        "sg_add_filter": ([vp, ctypes.POINTER(FilterDesc), ctypes.POINTER(i32)], ctypes.c_int),
        "sg_add_feedbackloop": ([vp, ctypes.POINTER(i32), ctypes.c_int, ctypes.POINTER(i32), i32, vp,
                                 ctypes.POINTER(i32)], ctypes.c_int),
        "sg_add_splitjoin": ([vp, ctypes.c_int, ctypes.POINTER(i32), ctypes.POINTER(i32), i32, ctypes.POINTER(i32)],
                             ctypes.c_int),
        "sg_branch_begin": ([vp, i32, i32], ctypes.c_int),
        "sg_branch_end": ([vp], ctypes.c_int),
        "sg_plan_opts_default": ([ctypes.POINTER(PlanOpts)], None),
        "sg_plan": ([vp, i32, ctypes.POINTER(PlanOpts), ctypes.POINTER(vp)], ctypes.c_int),
        "sg_input_items": ([vp, i64], i64),
        "sg_output_items": ([vp, i64], i64),
        "sg_plan_info": ([vp, ctypes.POINTER(PlanInfo)], ctypes.c_int),
        "sg_plan_source": ([vp, i32], ctypes.c_char_p),
        "sg_run": ([vp, vp, i64, vp, vp], ctypes.c_int),
        "sg_run_host": ([vp, vp, i64, vp], ctypes.c_int),
        "sg_last_launch_count": ([vp], i64),
        "sg_profile_partitions": ([vp, i64, i32, ctypes.POINTER(ctypes.c_double)], ctypes.c_int),
        "sg_plan_destroy": ([vp], None),
        "sg_last_error": ([], ctypes.c_char_p),
        "sg_version": ([], ctypes.c_char_p),
        "sg_flush_l2": ([vp, i64, vp], ctypes.c_int),
        "sg_topology_links": ([i32, i32], i32),
        "sg_topology_dtlist": ([i32, i32, ctypes.POINTER(ctypes.c_uint8)], ctypes.c_int),
        "sg_map_ilp": ([i32, ctypes.POINTER(ctypes.c_double), i32, ctypes.POINTER(i32), ctypes.POINTER(i32),
                        ctypes.POINTER(ctypes.c_double), i32, i32, ctypes.c_double, ctypes.c_double, i32, i32,
                        ctypes.POINTER(i32), ctypes.POINTER(ctypes.c_double), ctypes.POINTER(i32)], ctypes.c_int),
        "sg_paper_model": ([i32, ctypes.POINTER(ctypes.c_double), ctypes.POINTER(ctypes.c_double), i32, i32, i32,
                            ctypes.c_double, ctypes.c_double, ctypes.c_double, ctypes.POINTER(ctypes.c_double),
                            ctypes.POINTER(ctypes.c_double), ctypes.POINTER(ctypes.c_double)], ctypes.c_double),
        "sg_plan_pdg": ([vp, i32, ctypes.POINTER(i32), ctypes.POINTER(i32), ctypes.POINTER(ctypes.c_double)], i32),
        "sg_pee_features": ([vp, i32, ctypes.POINTER(ctypes.c_double), i32], i32),
        "sg_comm_unique_id": ([ctypes.POINTER(ctypes.c_uint8)], ctypes.c_int),
        "sg_comm_init": ([vp, i32, i32, ctypes.POINTER(ctypes.c_uint8), i32], ctypes.c_int),
        "sg_run_rank": ([vp, vp, i64, vp, vp], ctypes.c_int),
        "sg_rank_schedule": ([vp, i32, i64, ctypes.POINTER(RankOp), i64], i64),
    }
    for name, (args, res) in sig.items():
        fn = getattr(L, name)
        fn.argtypes = args
        fn.restype = res
    _lib = L
    return L


def _check(rc: int):
    if rc != SG_OK:
        raise SgError(rc, lib().sg_last_error().decode())


def _i32arr(v: Sequence[int]):
    return (ctypes.c_int32 * max(1, len(v)))(*v)


class Graph:
    """sg_graph handle.  Build with add_filter / splitjoin, or from a workloads Program."""

    def __init__(self, dtype: str = "f32"):
        self._h = ctypes.c_void_p()
        self.dtype = dtype
        _check(lib().sg_graph_create(SG_F32 if dtype == "f32" else SG_I32, ctypes.byref(self._h)))

    def add_filter(self, kind, ints=(), floats=()) -> int:
        k = KINDS[kind] if isinstance(kind, str) else int(kind)
        iv = _i32arr(list(ints))
        fv = (ctypes.c_float * max(1, len(floats)))(*floats)
        d = FilterDesc(k, len(ints), iv, len(floats), fv)
        eid = ctypes.c_int32(-1)
        _check(lib().sg_add_filter(self._h, ctypes.byref(d), ctypes.byref(eid)))
        return eid.value

    def add_splitjoin(self, dup: bool, n_branches: int, split_w=None, join_w=None) -> int:
        sj = ctypes.c_int32(-1)
        sw = _i32arr(split_w) if split_w is not None else None
        jw = _i32arr(join_w) if join_w is not None else None
        _check(lib().sg_add_splitjoin(self._h, 0 if dup else 1, sw, jw, n_branches, ctypes.byref(sj)))
        return sj.value

    def add_feedbackloop(self, join_w, dup: bool, split_w=None, enqueue=()) -> int:
        """Feedback loop; then fill branch 0 (body) and branch 1 (loop stream) with branch_begin/end."""
        lid = ctypes.c_int32(-1)
        jw = _i32arr(join_w)
        sw = _i32arr(split_w) if split_w is not None else None
        if self.dtype == "i32":
            enq = (ctypes.c_int32 * max(1, len(enqueue)))(*[int(v) for v in enqueue])
        else:
            enq = (ctypes.c_float * max(1, len(enqueue)))(*[float(v) for v in enqueue])
        _check(lib().sg_add_feedbackloop(self._h, jw, 0 if dup else 1, sw, len(enqueue), ctypes.cast(enq, ctypes.c_void_p),
                                         ctypes.byref(lid)))
        return lid.value

    def branch_begin(self, sj: int, b: int):
        _check(lib().sg_branch_begin(self._h, sj, b))

    def branch_end(self):
        _check(lib().sg_branch_end(self._h))

    def close(self):
        if self._h:
            lib().sg_graph_destroy(self._h)
            self._h = ctypes.c_void_p()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def graph_from_program(prog) -> Graph:
    """Marshal a neutral workloads.spec.Program into C-ABI builder calls."""
    from workloads.spec import FeedbackLoop, Filter, Pipeline  # neutral description, no arithmetic
    g = Graph(prog.dtype)

    def emit(s):
        if isinstance(s, Filter):
            g.add_filter(s.kind, s.ints, s.floats)
        elif isinstance(s, Pipeline):
            for c in s.children:
                emit(c)
        elif isinstance(s, FeedbackLoop):
            lid = g.add_feedbackloop(s.join_w, s.split == "dup", s.split_w, s.enqueue)
            for b, br in enumerate((s.body, s.loop)):
                g.branch_begin(lid, b)
                emit(br)
                g.branch_end()
        else:
            sj = g.add_splitjoin(s.split == "dup", len(s.branches), s.split_w, s.join_w)
            for b, br in enumerate(s.branches):
                g.branch_begin(sj, b)
                emit(br)
                g.branch_end()

    emit(prog.top)
    return g


class Plan:
    def __init__(self, graph, n_gpus: int = 1, **kw):
        own = False
        if not isinstance(graph, Graph):
            graph, own = graph_from_program(graph), True
        o = PlanOpts()
        lib().sg_plan_opts_default(ctypes.byref(o))
        self._keep = []
        for k, v in kw.items():
            if k == "node_partition":
                arr = _i32arr(v)
                self._keep.append(arr)
                o.node_partition = arr
                o.n_node_partition = len(v)
                o.partitioner = SG_PART_USER
            elif k == "devices":
                arr = _i32arr(v)
                self._keep.append(arr)
                o.devices = arr
            elif k == "codegen_mode" and isinstance(v, str):
                o.codegen_mode = {"auto": 0, "register": 1, "staged": 2, "general": 3}[v]
            elif k == "partitioner" and isinstance(v, str):
                o.partitioner = {"algorithm1": 0, "single": 1, "per_filter": 2, "chain": 4}[v]
            else:
                setattr(o, k, v)
        self._h = ctypes.c_void_p()
        try:
            _check(lib().sg_plan(graph._h, n_gpus, ctypes.byref(o), ctypes.byref(self._h)))
        finally:
            if own:
                graph.close()
        self.dtype = graph.dtype

    def info(self) -> dict:
        i = PlanInfo()
        _check(lib().sg_plan_info(self._h, ctypes.byref(i)))
        n, P = i.n_nodes, i.n_partitions
        return {
            "n_nodes": n, "n_edges": i.n_edges, "n_partitions": P, "n_gpus": i.n_gpus,
            "in_per_iter": i.in_per_iter, "out_per_iter": i.out_per_iter,
            "reps": [i.reps[k] for k in range(n)], "init_firings": [i.init_firings[k] for k in range(n)],
            "node_type": [i.node_type[k] for k in range(n)], "node_kind": [i.node_kind[k] for k in range(n)],
            "node_partition": [i.node_partition[k] for k in range(n)],
            "partition_gpu": [i.partition_gpu[k] for k in range(P)],
            "partition_time": [i.partition_time[k] for k in range(P)],
            "partition_mode": [i.partition_mode[k] for k in range(P)],
            "est_tmax": i.est_tmax, "input_device": i.input_device, "output_device": i.output_device,
            "iters_per_fragment": i.iters_per_fragment, "ilp_optimal": bool(i.ilp_optimal),
            "flops_per_iter_written": i.flops_per_iter_written, "flops_per_iter_pruned": i.flops_per_iter_pruned,
            "intops_per_iter": i.intops_per_iter,
            "replicas": i.replicas, "chain_fission": bool(i.chain_fission),
        }

    def input_items(self, n: int) -> int:
        v = lib().sg_input_items(self._h, n)
        if v < 0:
            _check(SG_E_ARG)
        return v

    def output_items(self, n: int) -> int:
        v = lib().sg_output_items(self._h, n)
        if v < 0:
            _check(SG_E_ARG)
        return v

    def source(self, part: int = 0) -> str:
        s = lib().sg_plan_source(self._h, part)
        return s.decode() if s else ""

    def run(self, x, n_iters: int, y, stream=None):
        """x, y: CUDA tensors (or raw device pointers); enqueued on `stream` (default: torch current stream)."""
        self._check_tensor(x, self.input_items(n_iters), "x")
        self._check_tensor(y, self.output_items(n_iters), "y")
        xp = x.data_ptr() if hasattr(x, "data_ptr") else int(x)
        yp = y.data_ptr() if hasattr(y, "data_ptr") else int(y)
        if stream is None:
            import torch
            stream = torch.cuda.current_stream().cuda_stream
        elif hasattr(stream, "cuda_stream"):
            stream = stream.cuda_stream
        _check(lib().sg_run(self._h, ctypes.c_void_p(xp), n_iters, ctypes.c_void_p(yp), ctypes.c_void_p(stream)))

    @staticmethod
    def _check_tensor(t, need: int, nm: str):
        """Tensors: on a CUDA device, contiguous, 4-byte items, at least `need` of them (raw pointers: unchecked)."""
        if not hasattr(t, "data_ptr"):
            return
        if not t.is_cuda:
            raise ValueError(f"{nm}: needs a CUDA tensor")
        if not t.is_contiguous() or t.element_size() != 4:
            raise ValueError(f"{nm}: needs a contiguous tensor of 4-byte items")
        if t.numel() < need:
            raise ValueError(f"{nm}: {t.numel()} items < {need} needed")

    def run_host(self, x, n_iters: int, y):
        """x, y: contiguous host numpy arrays (4-byte items); copies in, runs, copies out, synchronises."""
        for a, need, nm in ((x, self.input_items(n_iters), "x"), (y, self.output_items(n_iters), "y")):
            if a.dtype.itemsize != 4 or not a.flags["C_CONTIGUOUS"]:
                raise ValueError(f"{nm}: needs a C-contiguous array of 4-byte items")
            if a.size < need:
                raise ValueError(f"{nm}: {a.size} items < {need} needed for {n_iters} iterations")
        if not y.flags["WRITEABLE"]:
            raise ValueError("y: read-only array")
        _check(lib().sg_run_host(self._h, ctypes.c_void_p(x.ctypes.data), n_iters, ctypes.c_void_p(y.ctypes.data)))

    def pdg(self):
        n = lib().sg_plan_pdg(self._h, 0, None, None, None)
        a, b = (ctypes.c_int32 * max(1, n))(), (ctypes.c_int32 * max(1, n))()
        c = (ctypes.c_double * max(1, n))()
        lib().sg_plan_pdg(self._h, n, a, b, c)
        return [(a[i], b[i], c[i]) for i in range(n)]

    def rank_schedule(self, rank: int, n_iters: int):
        """Host-side op list sg_run_rank issues on `rank`: dicts with op/part/edge/peer/fragment/..."""
        cnt = lib().sg_rank_schedule(self._h, rank, n_iters, None, 0)
        if cnt < 0:
            raise SgError(SG_E_ARG, "bad rank / n_iters")
        buf = (RankOp * max(1, cnt))()
        lib().sg_rank_schedule(self._h, rank, n_iters, buf, cnt)
        return [{"op": o.op, "part": o.part, "edge": o.edge, "peer": o.peer, "fragment": o.fragment,
                 "k_begin": o.k_begin, "k_end": o.k_end, "items": o.items} for o in buf[:cnt]]

    def comm_init(self, nranks: int, rank: int, uid: bytes, device: int):
        arr = (ctypes.c_uint8 * 128)(*uid[:128])
        _check(lib().sg_comm_init(self._h, nranks, rank, arr, device))

    def run_rank(self, x, n_iters: int, y, stream=None):
        """One process per GPU: run this rank's partitions; x / y only on the input / output rank."""
        xp = 0 if x is None else (x.data_ptr() if hasattr(x, "data_ptr") else int(x))
        yp = 0 if y is None else (y.data_ptr() if hasattr(y, "data_ptr") else int(y))
        if stream is None:
            import torch
            stream = torch.cuda.current_stream().cuda_stream
        elif hasattr(stream, "cuda_stream"):
            stream = stream.cuda_stream
        _check(lib().sg_run_rank(self._h, ctypes.c_void_p(xp or None), n_iters, ctypes.c_void_p(yp or None),
                                 ctypes.c_void_p(stream)))

    def profile_partitions(self, n_iters: int, reps: int = 5):
        """Measured ns/iteration of every partition's kernel run alone (PEE validation, Fig. 4.1)."""
        k = self.info()["n_partitions"]
        buf = (ctypes.c_double * max(1, k))()
        _check(lib().sg_profile_partitions(self._h, n_iters, reps, buf))
        return [buf[i] for i in range(k)]

    PEE_FEATURES = ["mode", "flops", "intops", "dfma", "reads", "writes", "firings", "in_bytes", "out_bytes",
                    "levels", "halo_firings", "loop_firings", "cse_nodes", "frame", "bitslice", "est_ns",
                    "in_edges", "out_edges", "row_items", "fused", "tile", "threads", "smem", "source_bytes",
                    "reg_variant", "components", "fused_expected", "kernel_mode", "par_eff"]

    def pee_features(self, part: int) -> dict:
        """PEE inputs of one partition (work after the code generator's pruning / CSE, per iteration)."""
        buf = (ctypes.c_double * 29)()
        n = lib().sg_pee_features(self._h, part, buf, 29)
        if n < 0:
            raise SgError(SG_E_ARG, "bad partition")
        return {k: buf[i] for i, k in enumerate(self.PEE_FEATURES[:n])}

    def last_launch_count(self) -> int:
        return lib().sg_last_launch_count(self._h)

    def close(self):
        if getattr(self, "_h", None):
            lib().sg_plan_destroy(self._h)
            self._h = ctypes.c_void_p()

    def __enter__(self):
        return self

    def __exit__(self, *a):
        self.close()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def plan(program_or_graph, n_gpus: int = 1, **kw) -> Plan:
    return Plan(program_or_graph, n_gpus, **kw)


def flush_l2(scratch, stream=None):
    """Overwrite a device scratch tensor (> L2) with the nvcc-built sg_flush_l2 kernel."""
    if stream is None:
        import torch
        stream = torch.cuda.current_stream().cuda_stream
    _check(lib().sg_flush_l2(ctypes.c_void_p(scratch.data_ptr()), scratch.numel() * scratch.element_size(),
                             ctypes.c_void_p(stream)))


def topology_dtlist(kind: int, n_gpus: int):
    """dtlist[l][i][j] as nested lists (kind 0 NVSwitch star, 1 = PCIe tree of Fig. 3.3)."""
    L = lib().sg_topology_links(kind, n_gpus)
    if L < 0:
        raise SgError(SG_E_ARG, "bad topology")
    buf = (ctypes.c_uint8 * (L * n_gpus * n_gpus))()
    _check(lib().sg_topology_dtlist(kind, n_gpus, buf))
    G = n_gpus
    return [[[buf[l * G * G + i * G + j] for j in range(G)] for i in range(G)] for l in range(L)]


def map_ilp(T, edges, n_gpus, topo_kind=0, lat=0.0, bw=1.0, method=0, time_limit_ms=10000):
    """Solve Eq. III.1-III.7; edges = [(src, dst, bytes)].  Returns (assign, tmax, optimal)."""
    P = len(T)
    Ta = (ctypes.c_double * max(1, P))(*T)
    ne = len(edges)
    es = (ctypes.c_int32 * max(1, ne))(*[e[0] for e in edges])
    ed = (ctypes.c_int32 * max(1, ne))(*[e[1] for e in edges])
    eb = (ctypes.c_double * max(1, ne))(*[e[2] for e in edges])
    asg = (ctypes.c_int32 * max(1, P))()
    tm = ctypes.c_double(0)
    opt = ctypes.c_int32(0)
    _check(lib().sg_map_ilp(P, Ta, ne, es, ed, eb, topo_kind, n_gpus, lat, bw, time_limit_ms, method, asg,
                            ctypes.byref(tm), ctypes.byref(opt)))
    return [asg[i] for i in range(P)], tm.value, bool(opt.value)


def paper_model(t, f, S, W, F, D, C1=38.4, C2=11.2):
    """Eq. III.8-III.12; returns (T, Tcomp, Tdt, Tdb)."""
    n = len(t)
    ta = (ctypes.c_double * max(1, n))(*t)
    fa = (ctypes.c_double * max(1, n))(*f)
    a, b, c = ctypes.c_double(), ctypes.c_double(), ctypes.c_double()
    T = lib().sg_paper_model(n, ta, fa, S, W, F, D, C1, C2, ctypes.byref(a), ctypes.byref(b), ctypes.byref(c))
    return T, a.value, b.value, c.value


def comm_unique_id() -> bytes:
    arr = (ctypes.c_uint8 * 128)()
    _check(lib().sg_comm_unique_id(arr))
    return bytes(arr)


def version() -> str:
    return lib().sg_version().decode()
