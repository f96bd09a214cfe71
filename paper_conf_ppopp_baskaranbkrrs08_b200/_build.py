"""Build libsp.so in-tree: nvcc for sm_100a (-gencode arch=compute_100a,code=sm_100a).

The shared library is the product (C ABI in include/sp.h).  CUDA runtime is linked
statically; NCCL is dlopen-ed at run time (csrc/comm.cpp).  Everything is compiled with
-lineinfo so ncu's source page maps to the kernels, and without fast-math / FMA
contraction in the Jacobi translation unit (all its float ops are explicit .rn PTX).
"""
from __future__ import annotations

import os
import shutil
import subprocess
import sys

HERE = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(HERE)
CSRC = os.path.join(HERE, "csrc")
LIB = os.path.join(HERE, "libsp.so")
BUILD_DIR = os.path.join(ROOT, "build", "libsp")

SOURCES = ["api.cpp", "planner.cpp", "comm.cpp", "jacobi.cu", "me.cu", "ablation.cu", "exec.cu"]
HEADERS = ["sp_internal.h", "sm100_ptx.cuh", "sp_nccl_min.h"]
ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]


def nvcc() -> str:
    for cand in (os.environ.get("NVCC"), shutil.which("nvcc"), "/usr/local/cuda/bin/nvcc"):
        if cand and os.path.exists(cand):
            return cand
    raise RuntimeError("nvcc not found")


def _stale(target: str, deps: list[str]) -> bool:
    if not os.path.exists(target):
        return True
    t = os.path.getmtime(target)
    return any(os.path.getmtime(d) > t for d in deps)


def build(force: bool = False, verbose: bool = False) -> str:
    os.makedirs(BUILD_DIR, exist_ok=True)
    inc = os.path.join(ROOT, "include")
    hdrs = [os.path.join(CSRC, h) for h in HEADERS] + [os.path.join(inc, "sp.h")]
    objs = []
    for src in SOURCES:
        path = os.path.join(CSRC, src)
        obj = os.path.join(BUILD_DIR, src + ".o")
        objs.append(obj)
        if not force and not _stale(obj, [path, *hdrs]):
            continue
        cmd = [nvcc(), *ARCH, "-O3", "-lineinfo", "-std=c++17", "-I", inc, "-Xcompiler", "-fPIC,-O2,-ffp-contract=off",
               "-c", path, "-o", obj]
        if src.endswith(".cu"):
            cmd[1:1] = ["-Xptxas", "-v"] if verbose else []
            cmd += ["--fmad=false"]
        else:
            cmd[1:1] = ["-x", "c++"]
        if verbose:
            print(" ".join(cmd), file=sys.stderr)
        subprocess.check_call(cmd)
    if force or _stale(LIB, objs):
        tmp = LIB + f".tmp{os.getpid()}"
        cmd = [nvcc(), *ARCH, "-shared", "-o", tmp, *objs, "-cudart", "static", "-ldl", "-lpthread"]
        if verbose:
            print(" ".join(cmd), file=sys.stderr)
        subprocess.check_call(cmd)
        os.replace(tmp, LIB)
    return LIB


if __name__ == "__main__":
    build(force="--force" in sys.argv, verbose=True)
