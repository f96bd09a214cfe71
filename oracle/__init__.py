"""CPU oracle for the staged-tile hot path of Baskaran et al., PPoPP'08.

TEST INFRASTRUCTURE — NOT PART OF THE PRODUCT.  Only `tests/`,
`__graft_entry__.smoke()` and `bench.py`'s cpu_baseline / `--impl reference` legs may
import, call, link or execute anything under `oracle/`.  The product path
(`paper_conf_ppopp_baskaranbkrrs08_b200`) never imports it and fails loudly when its
CUDA extension is missing.  The oracle shares no code, headers, tables or constant
generators with the CUDA path; the only common module is `sp_inputs` (seeded input
generators, no method arithmetic).

Contents (each function cites the passage it follows, P = /root/reference/PAPER.md):
  oracle/oracle.c   — Jacobi 1-D (untiled definition, tiled twin, light-cone points,
                      fp64 twin) and exhaustive SAD motion estimation.
  oracle/planner.py — brute-force data-space enumeration for Alg. 1 / Alg. 2 / §3.1.2-3.

Pins (tests/test_oracle_*.py, `-m "not gpu"`): Figure 1's printed plan
(tests/golden/figure1.json), 1-D toy reuse cases, Jacobi fixed points (ramp, ones),
the fp64 sine-mode closed form, light cone, tiled == untiled, ME identical / shifted
frames, numpy-broadcast brute force, valid-candidate counts.  The paper's tile-size
optima and speedups are "parity unpinned" (context only).
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

from . import planner  # noqa: F401  (re-export)

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle.c")

# -O3 -march=native -ffp-contract=off, no -ffast-math (every fp32 op of the
# definition rounded as written; vectorisation keeps the op order).  -march=native ties the
# binary to the host CPU, so the library name carries a tag of the CPU model and flags: a box
# with another CPU builds its own copy instead of loading one it cannot execute.
CFLAGS = ["-O3", "-march=native", "-fopenmp", "-ffp-contract=off", "-fno-fast-math", "-fPIC", "-shared", "-std=c11"]


def cpu_model() -> str:
    try:
        with open("/proc/cpuinfo") as f:
            for ln in f:
                if ln.startswith("model name"):
                    return ln.split(":", 1)[1].strip()
    except OSError:
        pass
    return "unknown"


def _cpu_tag() -> str:
    import hashlib
    flags = ""
    try:
        with open("/proc/cpuinfo") as f:
            for ln in f:
                if ln.startswith("flags"):
                    flags = ln
                    break
    except OSError:
        pass
    return hashlib.sha1((cpu_model() + flags + " ".join(CFLAGS)).encode()).hexdigest()[:12]


_LIB = os.path.join(_HERE, f"liboracle.{_cpu_tag()}.so")


def build(force: bool = False) -> str:
    """Compile oracle.c into liboracle.<cpu tag>.so (gcc -O3 -march=native; no FMA contraction)."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        tmp = _LIB + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", *CFLAGS, "-o", tmp, _SRC])
        os.replace(tmp, _LIB)
    return _LIB


_lib = None


def lib():
    global _lib
    if _lib is None:
        build()
        L = ctypes.CDLL(_LIB)
        f32p = ctypes.POINTER(ctypes.c_float)
        f64p = ctypes.POINTER(ctypes.c_double)
        i64 = ctypes.c_int64
        i32 = ctypes.c_int32
        L.spo_set_threads.argtypes = [ctypes.c_int]
        L.spo_get_threads.restype = ctypes.c_int
        L.spo_jacobi1d.argtypes = [f32p, i64, i32, f32p]
        L.spo_jacobi1d_f64.argtypes = [f64p, i64, i32, f64p]
        L.spo_jacobi1d_tiled.argtypes = [f32p, i64, i32, i32, i64, f32p, f32p]
        L.spo_jacobi1d_points.argtypes = [f32p, i64, i32, ctypes.POINTER(i64), i64, f32p, f32p]
        L.spo_jacobi1d_window.argtypes = [f32p, i64, i64, i64, i32, f32p]
        L.spo_me_search.argtypes = [ctypes.c_void_p, ctypes.c_void_p, i64, i32, i32, i32,
                                    ctypes.POINTER(i32), i64, ctypes.POINTER(ctypes.c_int16),
                                    ctypes.POINTER(ctypes.c_uint32), ctypes.POINTER(ctypes.c_uint32)]
        L.spo_me_search_unrestricted.argtypes = L.spo_me_search.argtypes
        _lib = L
    return _lib


def _p(a: np.ndarray, ct):
    return a.ctypes.data_as(ctypes.POINTER(ct))


def set_threads(n: int) -> None:
    lib().spo_set_threads(int(n))


def get_threads() -> int:
    return int(lib().spo_get_threads())


def jacobi1d(a0: np.ndarray, steps: int) -> np.ndarray:
    """a^(steps) of the 1-D Jacobi recurrence (definition; oracle.c spo_jacobi1d)."""
    a = np.array(a0, dtype=np.float32, copy=True)
    work = np.empty_like(a)
    lib().spo_jacobi1d(_p(a, ctypes.c_float), a.size, int(steps), _p(work, ctypes.c_float))
    return a


def jacobi1d_f64(a0: np.ndarray, steps: int) -> np.ndarray:
    a = np.array(a0, dtype=np.float64, copy=True)
    work = np.empty_like(a)
    lib().spo_jacobi1d_f64(_p(a, ctypes.c_double), a.size, int(steps), _p(work, ctypes.c_double))
    return a


def jacobi1d_tiled(a0: np.ndarray, steps: int, time_tile: int, space_tile: int) -> np.ndarray:
    a = np.array(a0, dtype=np.float32, copy=True)
    work = np.empty_like(a)
    local = np.empty(2 * (space_tile + 2 * time_tile) + 8, dtype=np.float32)
    lib().spo_jacobi1d_tiled(_p(a, ctypes.c_float), a.size, int(steps), int(time_tile), int(space_tile),
                             _p(work, ctypes.c_float), _p(local, ctypes.c_float))
    return a


def jacobi1d_window(w: np.ndarray, g0: int, n: int, steps: int) -> np.ndarray:
    """h steps on a window holding global cells [g0, g0+len) (edges held; see oracle.c)."""
    a = np.array(w, dtype=np.float32, copy=True)
    scratch = np.empty_like(a)
    lib().spo_jacobi1d_window(_p(a, ctypes.c_float), a.size, int(g0), int(n), int(steps), _p(scratch, ctypes.c_float))
    return a


def jacobi1d_points(a0: np.ndarray, steps: int, idx) -> np.ndarray:
    a = np.ascontiguousarray(a0, dtype=np.float32)
    idx = np.ascontiguousarray(idx, dtype=np.int64)
    out = np.empty(idx.size, dtype=np.float32)
    scratch = np.empty(2 * (2 * int(steps) + 1) + 8, dtype=np.float32)
    lib().spo_jacobi1d_points(_p(a, ctypes.c_float), a.size, int(steps), _p(idx, ctypes.c_int64), idx.size,
                              _p(out, ctypes.c_float), _p(scratch, ctypes.c_float))
    return out


def me_search(ref: np.ndarray, cur: np.ndarray, width: int, height: int, search_range: int,
              mbs=None, with_surface: bool = False, unrestricted: bool = False):
    """Exhaustive SAD search of one (ref, cur) pair.  ref/cur: [height, pitch] uint8.
    Returns (mv [n,2] int16 (dx,dy), sad [n] uint32, surface [n,(2R+1)^2] or None)."""
    ref = np.ascontiguousarray(ref, dtype=np.uint8)
    cur = np.ascontiguousarray(cur, dtype=np.uint8)
    pitch = ref.shape[1]
    assert cur.shape[1] == pitch
    mbx, mby = width // 16, height // 16
    if mbs is None:
        mbs = np.arange(mbx * mby, dtype=np.int32)
    mbs = np.ascontiguousarray(mbs, dtype=np.int32)
    n = mbs.size
    mv = np.zeros((n, 2), dtype=np.int16)
    sad = np.zeros(n, dtype=np.uint32)
    side = 2 * search_range + 1
    surf = np.zeros((n, side * side), dtype=np.uint32) if with_surface else None
    fn = lib().spo_me_search_unrestricted if unrestricted else lib().spo_me_search
    fn(ref.ctypes.data, cur.ctypes.data, pitch, int(width), int(height), int(search_range),
       _p(mbs, ctypes.c_int32), n, _p(mv, ctypes.c_int16), _p(sad, ctypes.c_uint32),
       _p(surf, ctypes.c_uint32) if surf is not None else None)
    return mv, sad, surf
