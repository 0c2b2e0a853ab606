"""Build libsg.so in-tree (nvcc, sm_100a).

  python -m paper_conf_cgo_nguyenl16_b200.build [--force] [--precompile]

* sg_device.cuh is embedded as a string (sg_device_embed.inc) for NVRTC.
* Host C++ (graph IR, planner, code generator, runtime, C ABI) and the
  nvcc-compiled helper kernels (sg_aux.cu, -gencode arch=compute_100a,
  code=sm_100a) are linked into paper_conf_cgo_nguyenl16_b200/libsg.so
  against libnvrtc, libcuda (driver API) and libcudart.
* --precompile generates and NVRTC-compiles the kernels of the benchmark
  programs into the in-tree cubin cache (.sg_cache/), so a fresh GPU box
  loads them without compiling (pure cache; correctness never depends on it).
"""
from __future__ import annotations

import hashlib
import os
import subprocess
import sys

HERE = os.path.dirname(os.path.abspath(__file__))
CSRC = os.path.join(HERE, "csrc")
BUILD = os.path.join(HERE, "build")
LIB = os.path.join(HERE, "libsg.so")
CUDA = os.environ.get("CUDA_HOME", "/usr/local/cuda")
NVCC = os.path.join(CUDA, "bin", "nvcc")
ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]

CPP = ["sg_graph.cpp", "sg_codegen.cpp", "sg_pee.cpp", "sg_plan.cpp", "sg_runtime.cpp", "sg_dist.cpp", "sg_capi.cpp"]
CU = ["sg_aux.cu"]
HEADERS = ["sg_internal.h", "sg_codegen.h", "sg_runtime.h", "sg_plan.h", "sg_device.cuh"]


def _nccl_include():
    try:
        import nvidia.nccl
        d = os.path.join(list(nvidia.nccl.__path__)[0], "include")
        if os.path.exists(os.path.join(d, "nccl.h")):
            return d
    except Exception:
        pass
    return "/usr/include"


def _embed():
    src = open(os.path.join(CSRC, "sg_device.cuh")).read()
    assert ")SGDEV\"" not in src
    out = os.path.join(CSRC, "sg_device_embed.inc")
    text = 'R"SGDEV(' + src + ')SGDEV"\n'
    if not os.path.exists(out) or open(out).read() != text:
        with open(out, "w") as f:
            f.write(text)


def _deps_stamp():
    h = hashlib.sha256()
    for n in HEADERS + ["sg_device_embed.inc"]:
        h.update(open(os.path.join(CSRC, n), "rb").read())
    h.update(open(os.path.join(HERE, "..", "include", "sg.h"), "rb").read())
    return h.hexdigest()[:16]


def build(force: bool = False, verbose: bool = False) -> str:
    os.makedirs(BUILD, exist_ok=True)
    _embed()
    stamp = _deps_stamp()
    stamp_file = os.path.join(BUILD, "headers.stamp")
    if not os.path.exists(stamp_file) or open(stamp_file).read() != stamp:
        force = True
    objs = []
    for name in CPP + CU:
        src = os.path.join(CSRC, name)
        obj = os.path.join(BUILD, name + ".o")
        objs.append(obj)
        if not force and os.path.exists(obj) and os.path.getmtime(obj) >= os.path.getmtime(src):
            continue
        cmd = [NVCC, *ARCH, "-lineinfo", "-O3", "-std=c++17", "-Xcompiler", "-fPIC,-Wall,-Wno-array-bounds", "-c", src, "-o", obj,
               "-I" + os.path.join(HERE, "..", "include"), "-I" + _nccl_include()]
        if name.endswith(".cu"):
            cmd += ["-Xptxas", "-v"] if verbose else []
        else:
            cmd = [NVCC, "-x", "c++", *cmd[1:]]
        if verbose:
            print(" ".join(cmd))
        subprocess.check_call(cmd)
    need_link = force or not os.path.exists(LIB) or any(os.path.getmtime(o) > os.path.getmtime(LIB) for o in objs)
    if need_link:
        cmd = [NVCC, *ARCH, "-shared", "-o", LIB + ".tmp", *objs, "-L" + os.path.join(CUDA, "lib64"),
               "-L" + os.path.join(CUDA, "lib64", "stubs"), "-lnvrtc", "-lcudart",
               "-Xlinker", "-rpath," + os.path.join(CUDA, "lib64")]
        if verbose:
            print(" ".join(cmd))
        subprocess.check_call(cmd)
        os.replace(LIB + ".tmp", LIB)
    with open(stamp_file, "w") as f:
        f.write(stamp)
    return LIB


def precompile():
    """Plan the benchmark programs once (codegen + NVRTC, no GPU needed) to fill the cubin cache."""
    sys.path.insert(0, os.path.dirname(HERE))
    from workloads import apps
    from paper_conf_cgo_nguyenl16_b200 import sg
    for name, mk in {**apps.CONFIGS, **apps.EXTRA, **apps.FEEDBACK}.items():
        prog = mk()
        with sg.plan(prog, 1) as p:
            print(f"[precompile] {name}: {p.info()['n_partitions']} partition(s), modes {p.info()['partition_mode']}")


if __name__ == "__main__":
    build(force="--force" in sys.argv, verbose="-v" in sys.argv)
    print(LIB)
    if "--precompile" in sys.argv:
        precompile()
