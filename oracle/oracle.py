"""Python handle on the C oracle (oracle/sg_oracle.c) -- TEST INFRASTRUCTURE ONLY.

Only tests/, __graft_entry__.smoke() and bench.py (cpu_baseline leg and
--impl reference) may import this module.  The product package never does.

  build()                      compile liboracle.so with gcc (-O2 -ffp-contract=off)
  run(prog, x, n_iters)        sequential interpretation; returns the first
                               n_iters * out_per_iter output items
  rates(prog)                  repetition vector by exact balance equations
  in_items(prog, n_iters)      minimal input prefix producing n_iters iterations,
                               found by bisection over whole-program runs (a
                               definition, not a formula)
"""
from __future__ import annotations

import ctypes
import os
import subprocess
import threading

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "sg_oracle.c")
_LIB = os.path.join(_HERE, "liboracle.so")
_lock = threading.Lock()
_lib = None

T_FILTER, T_SPLIT_DUP, T_SPLIT_RR, T_JOIN_RR = 0, 1, 2, 3


def build(force: bool = False) -> str:
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        cmd = ["gcc", "-O2", "-ffp-contract=off", "-fno-fast-math", "-std=gnu11", "-shared", "-fPIC",
               "-o", _LIB + ".tmp", _SRC, "-lm"]
        subprocess.check_call(cmd)
        os.replace(_LIB + ".tmp", _LIB)
    return _LIB


def _get():
    global _lib
    with _lock:
        if _lib is None:
            build()
            lib = ctypes.CDLL(_LIB)
            lib.orc_run.argtypes = [ctypes.c_char_p, ctypes.c_void_p, ctypes.c_longlong, ctypes.c_void_p,
                                    ctypes.c_longlong, ctypes.POINTER(ctypes.c_longlong), ctypes.c_longlong,
                                    ctypes.c_int]
            lib.orc_run.restype = ctypes.c_int
            lib.orc_rates.argtypes = [ctypes.c_char_p, ctypes.POINTER(ctypes.c_longlong), ctypes.c_int,
                                      ctypes.POINTER(ctypes.c_int), ctypes.POINTER(ctypes.c_int),
                                      ctypes.POINTER(ctypes.c_longlong), ctypes.POINTER(ctypes.c_longlong)]
            lib.orc_rates.restype = ctypes.c_int
            _lib = lib
    return _lib


class OracleError(RuntimeError):
    def __init__(self, code):
        super().__init__(f"oracle error {code}")
        self.code = code


def _np_dtype(prog):
    return np.int32 if prog.dtype == "i32" else np.float32


def run_items(prog, x: np.ndarray, n_out: int, chunk: int = 4096, order_seed: int = 0) -> np.ndarray:
    """Run on the whole input `x`; return up to `n_out` output items."""
    lib = _get()
    x = np.ascontiguousarray(x, dtype=_np_dtype(prog))
    out = np.zeros(max(n_out, 1), dtype=_np_dtype(prog))
    got = ctypes.c_longlong(0)
    rc = lib.orc_run(prog.to_text().encode(), x.ctypes.data, x.size, out.ctypes.data, n_out,
                     ctypes.byref(got), chunk, order_seed)
    if rc:
        raise OracleError(rc)
    return out[: got.value]


def rates(prog) -> dict:
    lib = _get()
    maxn = 1 << 16
    reps = (ctypes.c_longlong * maxn)()
    info = (ctypes.c_int * (4 * maxn))()
    nn = ctypes.c_int(0)
    ipi = ctypes.c_longlong(0)
    opi = ctypes.c_longlong(0)
    rc = lib.orc_rates(prog.to_text().encode(), reps, maxn, ctypes.byref(nn), info, ctypes.byref(ipi),
                       ctypes.byref(opi))
    if rc:
        raise OracleError(rc)
    n = nn.value
    return {
        "reps": [reps[i] for i in range(n)],
        "type": [info[4 * i] for i in range(n)],
        "kind": [info[4 * i + 1] for i in range(n)],
        "pop": [info[4 * i + 2] for i in range(n)],
        "push": [info[4 * i + 3] for i in range(n)],
        "in_per_iter": ipi.value,
        "out_per_iter": opi.value,
    }


def run(prog, x: np.ndarray, n_iters: int, **kw) -> np.ndarray:
    """First n_iters * out_per_iter output items of the program on input x."""
    r = rates(prog)
    want = n_iters * r["out_per_iter"]
    y = run_items(prog, x, want, **kw)
    if y.size < want:
        raise ValueError(f"input too short: produced {y.size} of {want} items")
    return y


def in_items(prog, n_iters: int) -> int:
    """min L such that the program fed L items emits >= n_iters iterations of output."""
    if n_iters <= 0:
        return 0
    r = rates(prog)
    want = n_iters * r["out_per_iter"]

    def ok(L):
        x = np.zeros(L, dtype=_np_dtype(prog))
        return run_items(prog, x, want).size >= want

    if ok(0):
        return 0
    hi = max(1, n_iters * r["in_per_iter"])
    while not ok(hi):
        hi *= 2
    lo = 0  # ok(lo) is False for lo = 0 when want > 0
    while hi - lo > 1:
        mid = (lo + hi) // 2
        if ok(mid):
            hi = mid
        else:
            lo = mid
    return hi
