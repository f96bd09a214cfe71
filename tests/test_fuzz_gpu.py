"""Seeded random shapes through every device entry point, against the oracle (bit-exact).

The hand-picked edge shapes of the other GPU tests cover the known corners; this sweep
draws (n, steps, time tile, space tile, skew) and (frame size, range, pairs) at random so
shapes nobody thought of get exercised too.  Sizes stay small enough for the oracle."""
import numpy as np
import pytest
import torch

import oracle
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
import sp_inputs

pytestmark = pytest.mark.gpu


def _bits(x):
    return np.ascontiguousarray(x).view(np.uint32)


def _jacobi_cases(seed, count):
    rng = np.random.default_rng(seed)
    for _ in range(count):
        n = int(rng.integers(3, 60000))
        steps = int(rng.integers(0, 160))
        tt = int(rng.choice([1, 3, 8, 16, 17, 32, 64, 100, 128]))
        H = sp.halo_of(tt)
        s_max = sp.jacobi1d_plan(1 << 20, 64, tt, 0)["space_tile"]
        S = 0 if rng.random() < 0.4 else int(rng.integers(1, max(2, s_max // 4 + 1))) * 4
        S = min(S, s_max)
        yield n, steps, tt, S, H


@pytest.mark.parametrize("seed", range(8))
def test_jacobi_random_shapes_all_entry_points(seed, monkeypatch):
    checked = 0
    for n, steps, tt, S, H in _jacobi_cases(100 + seed, 6):
        checked += 1
        a0 = sp_inputs.jacobi_input(n, seed=seed * 1000 + n)
        want = _bits(oracle.jacobi1d(a0, steps))
        case = (n, steps, tt, S)
        d = torch.from_numpy(a0.copy()).cuda()
        sp.jacobi1d_timetiled(d, steps, tt, S)
        assert np.array_equal(_bits(d.cpu().numpy()), want), ("per-pass", case)
        for route in ("1", "0"):  # the persistent launch at every Tt; the default route (per pass below 16)
            monkeypatch.setenv("SP_JACOBI_FUSED_PERSISTENT", route)
            d = torch.from_numpy(a0.copy()).cuda()
            sp.jacobi1d_timetiled_fused(d, steps, tt, S)
            assert np.array_equal(_bits(d.cpu().numpy()), want), ("persistent" if route == "1" else "fused", case)
        if steps > 0:
            tiles = sp.jacobi1d_plan(n, steps, tt, S)["tiles"]
            reach = -(-H // (S if S else sp.jacobi1d_plan(n, steps, tt, 0)["space_tile"]))
            skew = 1
            while skew <= reach:
                skew *= 2
            skew *= int(np.random.default_rng(n).choice([1, 2, 8]))
            src = torch.from_numpy(a0.copy()).cuda()
            out = torch.empty_like(src)
            sp.jacobi1d_timetiled_stream(src, out, steps, tt, S, skew)
            assert np.array_equal(_bits(out.cpu().numpy()), want), ("wavefront", case, skew, tiles)
        h = torch.from_numpy(a0.copy()).pin_memory()
        sp.Jacobi1DHost(n, steps, tt, S).run(h)
        torch.cuda.synchronize()
        assert np.array_equal(_bits(h.numpy()), want), ("host", case)
        if n <= sp.jacobi1d_resident_capacity():
            src = torch.from_numpy(a0.copy()).cuda()
            out = sp.jacobi1d_resident(src, steps, out=torch.empty_like(src))
            assert np.array_equal(_bits(out.cpu().numpy()), want), ("resident", case)
    assert checked == 6


@pytest.mark.parametrize("seed", range(6))
def test_me_random_frames_surfaces(seed):
    rng = np.random.default_rng(200 + seed)
    pairs_checked = 0
    for _ in range(4):
        R = int(rng.choice([16, 32, 16, 32, 3, 9]))
        W = int(rng.integers(16, 200))
        H = int(rng.integers(16, 140))
        P = int(rng.integers(1, 4))
        pitch = (W + 15) // 16 * 16  # the device path needs 16-byte row pitch
        fr = sp_inputs.me_sequence(P + 1, W, H, R, pitch=pitch) if rng.random() < 0.5 else \
            sp_inputs.me_uniform_frames(P + 1, W, H, seed=int(rng.integers(1 << 30)), pitch=pitch)
        mv, sad, surf = sp.me_search_sequence(torch.from_numpy(fr).cuda(), W, H, R, with_surface=True)
        torch.cuda.synchronize()
        side = 2 * R + 1
        for p in range(P):
            omv, osad, osurf = oracle.me_search(fr[p], fr[p + 1], W, H, R, with_surface=True)
            case = (W, H, R, P, p)
            assert np.array_equal(mv[p].cpu().numpy().reshape(-1, 2), omv), case
            assert np.array_equal(_bits(sad[p].cpu().numpy()).reshape(-1), osad), case
            assert np.array_equal(_bits(surf[p].cpu().numpy()).reshape(-1, side * side), osurf), case
            pairs_checked += 1
    assert pairs_checked >= 4


@pytest.mark.parametrize("seed", range(6))
def test_me_random_frames_multi_wave(seed, monkeypatch):
    """Random frame sizes with more macroblocks than resident CTAs (each CTA then runs
    macroblocks from both pipeline stages), R in {16, 32}, the R = 16 class order with border
    searches forced on or off, and with a surface (every candidate's SAD, tails included)
    on every other draw; all pairs against the oracle."""
    rng = np.random.default_rng(900 + seed)
    R = 16 if seed % 3 else 32
    W = int(rng.integers(48, 360))
    H = int(rng.integers(48, 300))
    mbs = (W // 16) * (H // 16)
    P = max(2, -(-(3000 if R == 16 else 1200) // mbs))
    border = str(int(rng.integers(0, 2)))
    monkeypatch.setenv("SP_ME_BORDER", border)
    surface = seed % 2 == 1
    pitch = (W + 15) // 16 * 16
    fr = sp_inputs.me_sequence(P + 1, W, H, R, seed=int(rng.integers(1 << 30)), pitch=pitch)
    mv, sad, surf = sp.me_search_sequence(torch.from_numpy(fr).cuda(), W, H, R, with_surface=surface)
    torch.cuda.synchronize()
    side = 2 * R + 1
    for p in range(P):
        omv, osad, osurf = oracle.me_search(fr[p], fr[p + 1], W, H, R, with_surface=surface)
        case = (W, H, R, P, p, border, surface)
        assert np.array_equal(mv[p].cpu().numpy().reshape(-1, 2), omv), case
        assert np.array_equal(_bits(sad[p].cpu().numpy()).reshape(-1), osad), case
        if surface:
            assert np.array_equal(_bits(surf[p].cpu().numpy()).reshape(-1, side * side), osurf), case
