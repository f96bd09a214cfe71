"""Seeded synthetic input generators shared by the oracle side and the CUDA side.

This module holds NONE of the method's arithmetic (no stencil update, no SAD, no
footprint logic): it only produces inputs.  Both `oracle/` (via tests and
`bench.py`'s cpu_baseline leg) and the CUDA path (tests, bench, smoke) draw their
inputs from here, so the two sides see identical data without sharing any code.

Generators are counter-based (a pure function of seed and element coordinates),
so any shard of a workload can be regenerated independently by the rank that owns
it.

* Jacobi (BASELINE configs 1, 3, 5): a_i = 1 + (splitmix64(seed ^ i) >> 41) * 2^-23,
  an exactly representable fp32 value in [1, 2) for every cell, boundaries
  included.  Keeping |a| in [1, 2) keeps the relative-error metric well defined
  (reading R-J6).
* Motion estimation (BASELINE configs 2, 4): a 65-frame uint8 sequence whose frame f
  is a smooth periodic texture plus hash noise, displaced by a per-frame global pan
  and a per-region (4x4 regions) local offset in [-2, 2], plus +-2 per-frame noise
  (so consecutive-frame motion stays within [-R/2-4, R/2+4] ⊂ [-R, R] for R >= 8).  This gives
  the search the structure of real video (a dominant global motion, local
  deviations, texture ambiguity).  An i.i.d. uniform distribution is provided as a
  stress case.
"""
from __future__ import annotations

import math

import numpy as np

__all__ = [
    "splitmix64",
    "jacobi_input",
    "jacobi_ramp",
    "jacobi_ones",
    "jacobi_spike",
    "me_sequence",
    "me_frame",
    "me_uniform_frames",
    "me_shift_pair",
    "JACOBI_BENCH_SEED",
    "ME_BENCH_SEED",
]

JACOBI_BENCH_SEED = 2008
ME_BENCH_SEED = 2008

_M64 = np.uint64(0xFFFFFFFFFFFFFFFF)


def splitmix64(x: np.ndarray) -> np.ndarray:
    """SplitMix64 finaliser applied elementwise to a uint64 array (wrapping arithmetic)."""
    z = np.asarray(x, dtype=np.uint64)
    with np.errstate(over="ignore"):
        z = z + np.uint64(0x9E3779B97F4A7C15)
        z = (z ^ (z >> np.uint64(30))) * np.uint64(0xBF58476D1CE4E5B9)
        z = (z ^ (z >> np.uint64(27))) * np.uint64(0x94D049BB133111EB)
        z = z ^ (z >> np.uint64(31))
    return z


def jacobi_input(n: int, seed: int = JACOBI_BENCH_SEED, begin: int = 0, out: np.ndarray | None = None,
                 chunk: int = 1 << 24) -> np.ndarray:
    """Cells [begin, begin+n) of the seeded Jacobi initial state, float32 in [1, 2).

    a_i = 1 + (splitmix64(seed ^ i) >> 41) * 2^-23 (23 random mantissa bits).
    """
    if out is None:
        out = np.empty(n, dtype=np.float32)
    s = np.uint64(seed & 0xFFFFFFFFFFFFFFFF)
    for lo in range(0, n, chunk):
        hi = min(n, lo + chunk)
        idx = np.arange(begin + lo, begin + hi, dtype=np.uint64)
        m = (splitmix64(idx ^ s) >> np.uint64(41)).astype(np.uint32)
        # 1.0f has bit pattern 0x3F800000; OR-ing 23 mantissa bits gives 1 + m * 2^-23 exactly.
        out[lo:hi] = (m | np.uint32(0x3F800000)).view(np.float32)
    return out


def jacobi_ramp(n: int) -> np.ndarray:
    """a_i = i (exact fp32 fixed point of the 3-point average for n < 2^24/3)."""
    return np.arange(n, dtype=np.float32)


def jacobi_ones(n: int) -> np.ndarray:
    return np.ones(n, dtype=np.float32)


def jacobi_spike(n: int, at: int, value: float = 1.0) -> np.ndarray:
    a = np.zeros(n, dtype=np.float32)
    a[at] = value
    return a


# ---------------------------------------------------------------------------------------
# Motion-estimation frames
# ---------------------------------------------------------------------------------------

# Integer lookup tables for the smooth texture (periods 37 and 23 pixels).  They are
# computed once with math.sin/cos and rounded to integers, so every consumer sees the
# same integers.
_SIN37 = np.array([int(round(48.0 * math.sin(2.0 * math.pi * k / 37.0))) for k in range(37)], dtype=np.int64)
_COS23 = np.array([int(round(64.0 * math.cos(2.0 * math.pi * k / 23.0))) for k in range(23)], dtype=np.int64)


def _hash2(seed: int, tag: int, x: np.ndarray, y: np.ndarray) -> np.ndarray:
    """Counter-based 64-bit hash of (seed, tag, x, y) for int64 coordinate arrays."""
    xs = np.asarray(x, dtype=np.int64).astype(np.uint64)
    ys = np.asarray(y, dtype=np.int64).astype(np.uint64)
    with np.errstate(over="ignore"):
        k = (np.uint64((seed * 0x9E3779B1 + tag * 0x85EBCA77) & 0xFFFFFFFFFFFFFFFF)
             ^ (xs * np.uint64(0xD6E8FEB86659FD93))
             ^ (ys * np.uint64(0xA0761D6478BD642F)))
    return splitmix64(k)


def _texture(seed: int, x: np.ndarray, y: np.ndarray) -> np.ndarray:
    """Base texture T(x, y) for any integer coordinates (int64 arrays), int64 in [0,255]."""
    sx = _SIN37[np.mod(x, 37)]
    cy = _COS23[np.mod(y, 23)]
    noise = (_hash2(seed, 1, x, y) % np.uint64(81)).astype(np.int64) - 40
    v = 128 + (sx * cy) // 64 + noise
    return np.clip(v, 0, 255)


def _pan(seed: int, f: int, rng: int) -> tuple[int, int]:
    """Global pan between frame f and f+1, uniform in [-rng, rng]^2 (rng = R/2)."""
    h = int(_hash2(seed, 7, np.array([f]), np.array([0]))[0])
    span = 2 * rng + 1
    return (h % span) - rng, ((h >> 20) % span) - rng


def _region_offset(seed: int, f: int, rx: np.ndarray, ry: np.ndarray) -> tuple[np.ndarray, np.ndarray]:
    h = _hash2(seed, 11 + 2 * f, rx, ry)
    ox = (h % np.uint64(5)).astype(np.int64) - 2
    oy = ((h >> np.uint64(20)) % np.uint64(5)).astype(np.int64) - 2
    return ox, oy


def me_frame(f: int, width: int, height: int, search_range: int, seed: int = ME_BENCH_SEED,
             row_begin: int = 0, row_end: int | None = None) -> np.ndarray:
    """Rows [row_begin, row_end) of frame f of the synthetic sequence, uint8 [rows, width].

    frame_f(x, y) = T(x + Cx_f + ox_f(region), y + Cy_f + oy_f(region)) + e_f(x, y)
    where C_f is the cumulative global pan (each step uniform in [-R/2, R/2]), o_f the
    per-region offset in [-2, 2] over a 4x4 grid of regions, and e_f a +-2 noise.
    """
    if row_end is None:
        row_end = height
    rng = max(search_range // 2, 0)
    cx = cy = 0
    for g in range(f):
        px, py = _pan(seed, g, rng)
        cx += px
        cy += py
    ys = np.arange(row_begin, row_end, dtype=np.int64)[:, None]
    xs = np.arange(width, dtype=np.int64)[None, :]
    rx = (xs * 4) // max(width, 1)
    ry = (ys * 4) // max(height, 1)
    if f == 0:
        ox = np.zeros((1, 1), dtype=np.int64)
        oy = np.zeros((1, 1), dtype=np.int64)
    else:
        ox, oy = _region_offset(seed, f, np.broadcast_to(rx, (ys.shape[0], width)),
                                np.broadcast_to(ry, (ys.shape[0], width)))
    sx = xs + cx + ox
    sy = ys + cy + oy
    v = _texture(seed, np.broadcast_to(sx, (ys.shape[0], width)), np.broadcast_to(sy, (ys.shape[0], width)))
    if f > 0:
        e = (_hash2(seed, 1000 + f, np.broadcast_to(xs, v.shape), np.broadcast_to(ys, v.shape))
             % np.uint64(5)).astype(np.int64) - 2
        v = np.clip(v + e, 0, 255)
    return np.ascontiguousarray(v, dtype=np.uint8)


def me_sequence(n_frames: int, width: int, height: int, search_range: int, seed: int = ME_BENCH_SEED,
                pitch: int | None = None) -> np.ndarray:
    """[n_frames, height, pitch] uint8; columns >= width (row padding) are zero.

    Pair p of the batch is (ref = frame p, cur = frame p+1) (reading R-M6).
    """
    if pitch is None:
        pitch = width
    out = np.zeros((n_frames, height, pitch), dtype=np.uint8)
    for f in range(n_frames):
        out[f, :, :width] = me_frame(f, width, height, search_range, seed)
    return out


def me_uniform_frames(n_frames: int, width: int, height: int, seed: int = 1,
                      pitch: int | None = None) -> np.ndarray:
    """Stress distribution: i.i.d. uniform uint8 pixels."""
    if pitch is None:
        pitch = width
    out = np.zeros((n_frames, height, pitch), dtype=np.uint8)
    ys = np.arange(height, dtype=np.int64)[:, None]
    xs = np.arange(width, dtype=np.int64)[None, :]
    for f in range(n_frames):
        h = _hash2(seed, 5000 + f, np.broadcast_to(xs, (height, width)), np.broadcast_to(ys, (height, width)))
        out[f, :, :width] = (h & np.uint64(0xFF)).astype(np.uint8)
    return out


def me_shift_pair(width: int, height: int, shift_x: int, shift_y: int, seed: int = 3,
                  pitch: int | None = None) -> np.ndarray:
    """[2, height, pitch]: frame 0 = texture; frame 1 (cur) = frame 0 displaced so that
    cur(x, y) = ref(x + shift_x, y + shift_y) wherever the source lies inside the frame
    (outside: a different texture, so the true vector is only guaranteed inside)."""
    if pitch is None:
        pitch = width
    ys = np.arange(height, dtype=np.int64)[:, None]
    xs = np.arange(width, dtype=np.int64)[None, :]
    X = np.broadcast_to(xs, (height, width))
    Y = np.broadcast_to(ys, (height, width))
    ref = _texture(seed, X, Y)
    cur = _texture(seed, X + shift_x, Y + shift_y)
    out = np.zeros((2, height, pitch), dtype=np.uint8)
    out[0, :, :width] = ref
    out[1, :, :width] = cur
    return out
