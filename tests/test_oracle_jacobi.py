"""Pins for the Jacobi oracle (oracle/oracle.c) against what the mathematics fixes.

Reading R-J1: a^(t+1)_i = fl(fl(fl(a_{i-1} + a_i) + a_{i+1}) * w), w = fl32(1/3),
1 <= i <= N-2, a_0 and a_{N-1} fixed; P:L859-862, L960-967 (the paper never prints the
statement).  Each pin below fails under a plausible mistake: a dropped or shifted
neighbour, a wrong weight, updating the boundary, an off-by-one step count.
"""
import math

import numpy as np
import pytest

import oracle
import sp_inputs

U = 2.0 ** -24  # unit roundoff of fp32


def test_weight_is_fl32_one_third():
    # the oracle's w: a spike of 1.0 after one step gives w at its three cells
    a = sp_inputs.jacobi_spike(7, 3)
    r = oracle.jacobi1d(a, 1)
    assert r[2] == r[3] == r[4] == np.float32(1.0) / np.float32(3.0)
    assert np.float32(1.0 / 3.0).view(np.uint32) == 0x3EAAAAAB
    assert r[0] == r[1] == r[5] == r[6] == 0.0


def test_ramp_is_exact_fixed_point():
    # a_i = i: 3i is exact, and fl(3i * w) = i since 3i*w = i(1 + 2^-25) rounds back to i.
    a = sp_inputs.jacobi_ramp(4096)
    assert np.array_equal(oracle.jacobi1d(a, 64), a)
    assert np.array_equal(oracle.jacobi1d(a, 7), a)


def test_ones_is_exact_fixed_point():
    a = sp_inputs.jacobi_ones(1000)
    assert np.array_equal(oracle.jacobi1d(a, 50), a)


def test_zero_steps_is_identity_and_boundaries_fixed():
    a = sp_inputs.jacobi_input(513, seed=1)
    assert np.array_equal(oracle.jacobi1d(a, 0), a)
    r = oracle.jacobi1d(a, 17)
    assert r[0] == a[0] and r[-1] == a[-1]
    assert not np.array_equal(r[1:-1], a[1:-1])


def _sine_mode(n, k):
    i = np.arange(n, dtype=np.float64)
    a = np.sin(math.pi * k * i / (n - 1))
    a[0] = 0.0
    a[-1] = 0.0
    lam = (1.0 + 2.0 * math.cos(math.pi * k / (n - 1))) / 3.0
    return a, lam


@pytest.mark.parametrize("k", [1, 3, 17])
def test_fp64_twin_matches_eigenmode_closed_form(k):
    # sin(pi k i/(N-1)) is an eigenvector of the 3-point average with zero Dirichlet ends:
    # (sin(x-h) + sin x + sin(x+h))/3 = sin x (1 + 2 cos h)/3.
    n, T = 513, 64
    a, lam = _sine_mode(n, k)
    got = oracle.jacobi1d_f64(a, T)
    assert np.max(np.abs(got - lam ** T * a)) < 1e-12


@pytest.mark.parametrize("k", [1, 5])
def test_fp32_oracle_within_rounding_bound_of_closed_form(k):
    # per step: two rounded adds, one rounded multiply, and |w - 1/3| <= (1/3) 2^-24, and the
    # averaging operator is non-expansive in max-norm, so the accumulated error is at most
    # (4T + 1) u max|a| (the +1 is the initial rounding to fp32).
    n, T = 4096, 64
    a, lam = _sine_mode(n, k)
    got = oracle.jacobi1d(a.astype(np.float32), T).astype(np.float64)
    err = np.max(np.abs(got - lam ** T * a))
    assert err <= (4 * T + 1) * U * 1.0
    # a real (not vacuous) check: a shifted stencil would be off by O(1e-3) here
    assert err < 1e-4


def test_light_cone_and_front_value():
    # a spike at c: after T steps the support is exactly [c-T, c+T] and the front cell
    # holds w^T computed by T successive fp32 multiplications (the only path reaching it).
    n, c, T = 301, 150, 40
    r = oracle.jacobi1d(sp_inputs.jacobi_spike(n, c), T)
    nz = np.nonzero(r)[0]
    assert nz.min() == c - T and nz.max() == c + T
    w = np.float32(1.0) / np.float32(3.0)
    v = np.float32(1.0)
    for _ in range(T):
        v = np.float32(v * w)
    assert r[c + T] == v and r[c - T] == v


def test_tiled_twin_equals_untiled_bit_exact():
    # overlapped time tiling with owned-region write-back (R-J4, R-J5) is exact
    for (n, T, tt, s) in [(4096, 64, 16, 256), (1000, 37, 16, 64), (50, 9, 4, 7), (3, 5, 2, 1), (777, 33, 32, 100)]:
        a = sp_inputs.jacobi_input(n, seed=2)
        assert np.array_equal(oracle.jacobi1d_tiled(a, T, tt, s), oracle.jacobi1d(a, T)), (n, T, tt, s)


def test_points_sampler_equals_full_result():
    n, T = 2000, 50
    a = sp_inputs.jacobi_input(n, seed=3)
    full = oracle.jacobi1d(a, T)
    idx = np.array([0, 1, 2, 49, 50, 51, 999, 1948, 1949, 1950, 1998, 1999])
    assert np.array_equal(oracle.jacobi1d_points(a, T, idx), full[idx])


def test_generator_values_exact_in_unit_interval():
    a = sp_inputs.jacobi_input(1 << 16, seed=2008)
    assert a.dtype == np.float32 and a.min() >= 1.0 and a.max() < 2.0
    # 23 random mantissa bits: every value is 1 + m 2^-23 exactly
    m = (a.astype(np.float64) - 1.0) * 2 ** 23
    assert np.array_equal(m, np.round(m))
    # counter-based: a shard regenerates identically
    assert np.array_equal(sp_inputs.jacobi_input(100, seed=2008, begin=5000), a[5000:5100])
