"""Direct pins for the window form of the Jacobi oracle (oracle.c spo_jacobi1d_window): h steps
of the definition (reading R-J1) on a window [g0, g0 + len) of an
n-cell domain, the window's own edge cells held fixed (their true neighbours lie outside), the
domain's boundary cells 0 and n - 1 fixed.  It is the per-rank compute of the gloo
decomposition test (tests/test_dist_gloo.py).  Each pin fails under a plausible mistake: a
wrong weight or op order, a shifted neighbour, an updated window edge or domain boundary, a
light cone that leaks (reading beyond the window), an off-by-one step count."""
import numpy as np
import pytest

import oracle
import sp_inputs

W = np.float32(1.0) / np.float32(3.0)  # fl32(1/3) = 0x3EAAAAAB


def test_spike_one_step_gives_w_on_three_cells():
    w = np.zeros(11, np.float32)
    w[5] = 1.0
    r = oracle.jacobi1d_window(w, 100, 1000, 1)  # an interior window of a large domain
    assert r[4] == r[5] == r[6] == W
    assert np.all(r[[1, 2, 3, 7, 8, 9]] == 0) and r[0] == 0 and r[10] == 0


@pytest.mark.parametrize("steps", [1, 4, 9])
def test_light_cone_front_is_iterated_product(steps):
    # a spike's front after t steps is fl(...fl(fl(v w) w)... w): (0 + 0) + x = x exactly,
    # so the cell at distance t from the spike is w multiplied in t times, rounded each time
    v = np.float32(1.75)
    w = np.zeros(41, np.float32)
    w[20] = v
    r = oracle.jacobi1d_window(w, 500, 10_000, steps)
    front = v
    for _ in range(steps):
        front = np.float32(front * W)
    assert r[20 + steps] == front and r[20 - steps] == front
    assert np.all(r[20 + steps + 1:] == 0) and np.all(r[:20 - steps] == 0)


def test_ramp_window_is_fixed_point():
    # a_i = i is an exact fixed point of the update (3i exact, fl(3i w) = i for 3i < 2^24);
    # window edges are held, so the whole window stays the ramp for any number of steps
    g0, n = 3000, 100_000
    w = np.arange(g0, g0 + 257, dtype=np.float32)
    assert np.array_equal(oracle.jacobi1d_window(w, g0, n, 40), w)


def test_window_edges_and_domain_boundaries_stay_fixed():
    w = sp_inputs.jacobi_input(64, seed=3)
    r = oracle.jacobi1d_window(w, 500, 10_000, 7)  # interior window: its two edge cells held
    assert r[0] == w[0] and r[-1] == w[-1]
    assert not np.array_equal(r[1:-1], w[1:-1])
    r0 = oracle.jacobi1d_window(w, 0, 64, 7)       # the whole domain: global cells 0 and 63 fixed
    assert r0[0] == w[0] and r0[-1] == w[-1]
    # a window at the domain's left end whose last cell is global n - 1
    r1 = oracle.jacobi1d_window(w, 10_000 - 64, 10_000, 7)
    assert r1[-1] == w[-1]


def test_no_dependence_beyond_the_light_cone():
    # after h steps, cell j depends only on cells within distance h of it
    w = sp_inputs.jacobi_input(101, seed=4)
    h = 6
    base = oracle.jacobi1d_window(w, 1000, 100_000, h)
    for far in (50 + h + 1, 50 - h - 1, 0, 100):
        p = w.copy()
        p[far] = np.float32(1.5) if p[far] != 1.5 else np.float32(1.25)
        assert oracle.jacobi1d_window(p, 1000, 100_000, h)[50] == base[50]
    p = w.copy()
    p[50 + h] += np.float32(0.5)  # inside the cone: the result must change
    assert oracle.jacobi1d_window(p, 1000, 100_000, h)[50] != base[50]


def test_zero_steps_is_identity():
    w = sp_inputs.jacobi_input(33, seed=5)
    assert np.array_equal(oracle.jacobi1d_window(w, 7, 1000, 0), w)
