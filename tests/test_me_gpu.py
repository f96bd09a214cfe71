"""GPU parity of the motion-estimation path (libsp sp_me_sad_search) against the CPU
oracle (oracle.me_search) on the same seeded frames: motion vectors, best SADs and the
full SAD surface must be bit-identical (integer work)."""
import numpy as np
import pytest
import torch

import oracle
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
import sp_inputs

pytestmark = pytest.mark.gpu


def _pitch(w):
    return (w + 15) // 16 * 16


def _gpu(frames, W, H, R, **kw):
    d = torch.from_numpy(frames).cuda()
    mv, sad, surf = sp.me_search_sequence(d, W, H, R, **kw)
    torch.cuda.synchronize()
    return mv.cpu().numpy(), sad.cpu().numpy().view(np.uint32), None if surf is None else surf.cpu().numpy().view(np.uint32)


def _oracle_pair(frames, p, W, H, R, surface=True, mbs=None):
    return oracle.me_search(frames[p], frames[p + 1], W, H, R, mbs=mbs, with_surface=surface)


@pytest.mark.parametrize("gen", ["seq", "uniform"])
def test_M2_cif_full_surface(gen):
    # BASELINE config 2: CIF 352x288, 16x16 MBs, +-16
    W, H, R = 352, 288, 16
    fr = sp_inputs.me_sequence(3, W, H, R) if gen == "seq" else sp_inputs.me_uniform_frames(3, W, H, seed=2)
    mv, sad, surf = _gpu(fr, W, H, R, with_surface=True)
    for p in range(2):
        omv, osad, osurf = _oracle_pair(fr, p, W, H, R)
        assert np.array_equal(mv[p].reshape(-1, 2), omv)
        assert np.array_equal(sad[p].reshape(-1), osad)
        assert np.array_equal(surf[p].reshape(osurf.shape), osurf)


@pytest.mark.parametrize("W,H", [(16, 16), (40, 36), (64, 48), (100, 70), (129, 47)])
@pytest.mark.parametrize("R", [0, 1, 2, 5, 8, 16, 24, 32])
def test_small_frames_all_ranges(W, H, R):
    fr = sp_inputs.me_sequence(2, W, H, max(R, 2), seed=W + R, pitch=_pitch(W))
    mv, sad, surf = _gpu(fr, W, H, R, with_surface=True)
    omv, osad, osurf = _oracle_pair(fr, 0, W, H, R)
    assert np.array_equal(mv[0].reshape(-1, 2), omv)
    assert np.array_equal(sad[0].reshape(-1), osad)
    assert np.array_equal(surf[0].reshape(osurf.shape), osurf)


def test_identical_and_flat_and_shifted():
    W, H, R = 96, 80, 16
    fr = sp_inputs.me_sequence(1, W, H, R)
    same = np.concatenate([fr, fr])
    mv, sad, _ = _gpu(same, W, H, R)
    assert np.all(mv == 0) and np.all(sad == 0)
    flat = np.stack([np.full((H, W), 9, np.uint8), np.full((H, W), 200, np.uint8)])
    mv, sad, _ = _gpu(flat, W, H, R)
    assert np.all(mv == 0) and np.all(sad == 256 * 191)
    sh = sp_inputs.me_shift_pair(W, H, 5, -3)
    mv, sad, _ = _gpu(sh, W, H, R)
    omv, osad, _ = _oracle_pair(sh, 0, W, H, R, surface=False)
    assert np.array_equal(mv[0].reshape(-1, 2), omv) and np.array_equal(sad[0].reshape(-1), osad)


def test_band_equals_full_frame():
    """A rank's band (MB rows [4, 9) with an R-row halo) gives the same result as the
    full-frame search for those rows (multi-GPU sharding building block)."""
    from paper_conf_ppopp_baskaranbkrrs08_b200.partition import me_band_rows
    W, H, R = 352, 288, 16
    fr = sp_inputs.me_sequence(3, W, H, R)
    full_mv, full_sad, _ = _gpu(fr, W, H, R)
    r0, r1 = me_band_rows(4, 9, H, R)
    band = np.ascontiguousarray(fr[:, r0:r1])
    d = torch.from_numpy(band).cuda()
    mv, sad, _ = sp.me_sad_search(d[:-1], d[1:], W, H, R, row0=r0, mb_row_begin=4, mb_row_end=9)
    torch.cuda.synchronize()
    assert np.array_equal(mv.cpu().numpy(), full_mv[:, 4:9])
    assert np.array_equal(sad.cpu().numpy().view(np.uint32), full_sad[:, 4:9])


def test_M4_1080p_sampled():
    """BASELINE config 4 (1920x1080, +-32, 64 pairs) in the bench launch configuration;
    oracle on sampled macroblocks of every pair (all border MBs of pairs 0 and 63, plus
    random MBs everywhere)."""
    W, H, R, F = 1920, 1080, 32, 65
    fr = sp_inputs.me_sequence(F, W, H, R)
    mv, sad, _ = _gpu(fr, W, H, R)
    mbx, mby = W // 16, H // 16
    rng = np.random.default_rng(1)
    border = [by * mbx + bx for by in range(mby) for bx in range(mbx) if by in (0, mby - 1) or bx in (0, mbx - 1)]
    for p in range(F - 1):
        mbs = rng.choice(mbx * mby, 6, replace=False).tolist()
        if p in (0, F - 2):
            mbs += border
        mbs = np.array(sorted(set(mbs)), dtype=np.int32)
        omv, osad, _ = _oracle_pair(fr, p, W, H, R, surface=False, mbs=mbs)
        assert np.array_equal(mv[p].reshape(-1, 2)[mbs], omv), p
        assert np.array_equal(sad[p].reshape(-1)[mbs], osad), p


def test_M4_1080p_every_macroblock_device_and_host_paths():
    """BASELINE config 4 in full: every macroblock of all 64 pairs (2,107,814,400 valid
    candidate SADs) from the bench's launch (device-resident frames) and from the end-to-end
    host-buffer call (streamed frames, outputs in pinned memory), against the oracle on all
    of them (about 2 s of host time on 16 cores)."""
    W, H, R, F = 1920, 1080, 32, 65
    fr = sp_inputs.me_sequence(F, W, H, R)
    mv, sad, _ = _gpu(fr, W, H, R)
    ctx = sp.MESearchHost(F, W, H, fr.shape[2], R)
    hmv, hsad = ctx.run(torch.from_numpy(fr).pin_memory())
    torch.cuda.synchronize()
    hmv, hsad = hmv.numpy(), hsad.numpy().view(np.uint32)
    for p in range(F - 1):
        omv, osad, _ = _oracle_pair(fr, p, W, H, R, surface=False)
        assert np.array_equal(mv[p].reshape(-1, 2), omv), p
        assert np.array_equal(sad[p].reshape(-1), osad), p
        assert np.array_equal(hmv[p].reshape(-1, 2), omv), p
        assert np.array_equal(hsad[p].reshape(-1), osad), p


def test_host_api_end_to_end():
    W, H, R = 352, 288, 16
    fr = sp_inputs.me_sequence(4, W, H, R)
    mv, sad = sp.me_search(fr, W, H, R)
    omv, osad, _ = _oracle_pair(fr, 2, W, H, R, surface=False)
    assert np.array_equal(mv[2].numpy().reshape(-1, 2), omv)
    assert np.array_equal(sad[2].numpy().view(np.uint32).reshape(-1), osad)


@pytest.mark.parametrize("W,H,R", [(64, 48, 5), (352, 288, 16), (130, 70, 32), (64, 64, 32)])
def test_unrestricted_equals_oracle(W, H, R):
    fr = sp_inputs.me_sequence(3, W, H, max(R, 2), seed=12, pitch=_pitch(W))
    d = torch.from_numpy(fr).cuda()
    mv, sad, surf = sp.me_search_sequence_unrestricted(d, W, H, R, with_surface=True)
    torch.cuda.synchronize()
    for p in range(2):
        omv, osad, osurf = oracle.me_search(fr[p], fr[p + 1], W, H, R, with_surface=True, unrestricted=True)
        assert np.array_equal(mv[p].cpu().numpy().reshape(-1, 2), omv)
        assert np.array_equal(sad[p].cpu().numpy().view(np.uint32).reshape(-1), osad)
        assert np.array_equal(surf[p].cpu().numpy().view(np.uint32).reshape(osurf.shape), osurf)


def test_pad_frames_edge_extension():
    W, H, pad = 50, 30, 16
    fr = sp_inputs.me_uniform_frames(2, W, H, seed=4, pitch=64)
    out = sp.me_pad_frames(torch.from_numpy(fr).cuda(), W, H, pad).cpu().numpy()
    for f in range(2):
        want = np.pad(fr[f, :, :W], pad, mode="edge")
        assert np.array_equal(out[f, :, :W + 2 * pad], want)


@pytest.mark.parametrize("W,H", [(96, 80), (352, 288), (64, 64), (48, 32), (100, 70), (160, 96), (16, 48), (80, 16),
                                 (129, 47), (208, 144)])
@pytest.mark.parametrize("R", [16, 32])
@pytest.mark.parametrize("gen", ["seq", "uniform", "flat"])
def test_border_macroblocks_without_surface(W, H, R, gen):
    """MVs and SADs without a surface (the bench's launch form) on frames whose border
    macroblocks have few valid candidates: sides multiples of 16 or not, tiny frames where both
    sides bind, flat frames (every candidate ties: the tie-break across the main block, the
    tails and the corner candidate)."""
    pitch = _pitch(W)
    if gen == "seq":
        fr = sp_inputs.me_sequence(3, W, H, R, seed=W * 3 + H + R, pitch=pitch)
    elif gen == "uniform":
        fr = sp_inputs.me_uniform_frames(3, W, H, seed=W + H, pitch=pitch)
    else:
        fr = np.zeros((3, H, pitch), np.uint8)
        fr[0], fr[1], fr[2] = 7, 7, 200
    mv, sad, _ = _gpu(fr, W, H, R)
    for p in range(2):
        omv, osad, _ = _oracle_pair(fr, p, W, H, R, surface=False)
        assert np.array_equal(mv[p].reshape(-1, 2), omv), p
        assert np.array_equal(sad[p].reshape(-1), osad), p


@pytest.mark.parametrize("W,H", [(352, 288), (96, 80), (48, 48), (100, 70), (129, 47), (64, 40), (360, 280)])
@pytest.mark.parametrize("gen", ["seq", "flat"])
@pytest.mark.parametrize("border", ["1", "0"])
def test_class_order_border_search(W, H, gen, border, monkeypatch):
    """R = 16 class order (interior macroblocks of every pair first, then rows, columns,
    corners) with half-frame border searches, forced on ($SP_ME_BORDER=1) and off, against the
    oracle on every macroblock of several pairs: sides multiples of 16 or not (then the last
    row / column keeps the full search inside the border phase), 3 x 3 macroblock frames
    (one interior macroblock), flat frames (ties across the moved tails and corner)."""
    R = 16
    monkeypatch.setenv("SP_ME_BORDER", border)
    pitch = _pitch(W)
    if gen == "seq":
        fr = sp_inputs.me_sequence(6, W, H, R, seed=W * 7 + H, pitch=pitch)
    else:
        fr = np.zeros((6, H, pitch), np.uint8)
        fr[0::2], fr[1::2] = 7, 200
        fr[2] = 9
    mv, sad, _ = _gpu(fr, W, H, R)
    for p in range(5):
        omv, osad, _ = _oracle_pair(fr, p, W, H, R, surface=False)
        assert np.array_equal(mv[p].reshape(-1, 2), omv), p
        assert np.array_equal(sad[p].reshape(-1), osad), p


@pytest.mark.parametrize("R", [16, 32])
def test_many_macroblocks_per_cta_full_surface(R):
    """More macroblocks than resident CTAs (8 CIF pairs at R = 16: 3,168 macroblocks on
    2,368 one-warp CTAs; 40 pairs at R = 32), so CTAs run a second macroblock from the other
    pipeline stage: every SAD of every candidate, tails included, equals the oracle.  (Until
    round-2 session 3 the one-warp R = 16 kernel read byte-phase-0 tails from stage 0's window
    on every macroblock; single-wave tests could not see it.)"""
    W, H = 352, 288
    P = 8 if R == 16 else 40
    fr = sp_inputs.me_sequence(P + 1, W, H, R, seed=5 + R)
    mv, sad, surf = _gpu(fr, W, H, R, with_surface=True)
    for p in range(P):
        omv, osad, osurf = _oracle_pair(fr, p, W, H, R)
        assert np.array_equal(surf[p].reshape(osurf.shape), osurf), p
        assert np.array_equal(mv[p].reshape(-1, 2), omv), p
        assert np.array_equal(sad[p].reshape(-1), osad), p


def test_class_order_auto_many_pairs():
    """The automatic class order (>= 8192 macroblocks: 24 CIF pairs) on the R = 16 throughput
    form: every macroblock of every pair equals the oracle."""
    W, H, R, P = 352, 288, 16, 24
    fr = sp_inputs.me_sequence(P + 1, W, H, R, seed=77)
    mv, sad, _ = _gpu(fr, W, H, R)
    for p in range(P):
        omv, osad, _ = _oracle_pair(fr, p, W, H, R, surface=False)
        assert np.array_equal(mv[p].reshape(-1, 2), omv), p
        assert np.array_equal(sad[p].reshape(-1), osad), p


def test_prepared_call_equals_oracle():
    """me_search_prepared (arguments marshalled once, the latency-config call form) runs the
    same entry point: repeated calls give the oracle's MVs / SADs."""
    W, H, R = 352, 288, 16
    fr = sp_inputs.me_sequence(3, W, H, R, seed=41)
    call = sp.me_search_prepared(torch.from_numpy(fr).cuda(), W, H, R)
    for _ in range(3):
        call()
    torch.cuda.synchronize()
    for p in range(2):
        omv, osad, _ = _oracle_pair(fr, p, W, H, R, surface=False)
        assert np.array_equal(call.mv[p].cpu().numpy().reshape(-1, 2), omv)
        assert np.array_equal(call.sad[p].cpu().numpy().view(np.uint32).reshape(-1), osad)
