"""GPU parity of the end-to-end host-buffer motion estimation (sp_me_search_host): frames
streamed frame by frame into device memory while the search runs (ready flags), MV / SAD
stored by the kernel into pinned host memory (or device memory).  Bit-exact against the
oracle and against the device-resident path."""
import numpy as np
import pytest
import torch

import oracle
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
import sp_inputs

pytestmark = pytest.mark.gpu


def _device_path(frames, W, H, R):
    mv, sad, _ = sp.me_search_sequence(torch.from_numpy(frames).cuda(), W, H, R)
    torch.cuda.synchronize()
    return mv.cpu().numpy(), sad.cpu().numpy()


@pytest.mark.parametrize("gen", ["seq", "uniform"])
def test_cif_sequence_vs_oracle(gen):
    W, H, R = 352, 288, 16
    fr = sp_inputs.me_sequence(5, W, H, R) if gen == "seq" else sp_inputs.me_uniform_frames(5, W, H, seed=4)
    mv, sad = sp.me_search(fr, W, H, R)
    mv, sad = mv.numpy(), sad.numpy().view(np.uint32)
    for p in range(4):
        omv, osad, _ = oracle.me_search(fr[p], fr[p + 1], W, H, R)
        assert np.array_equal(mv[p].reshape(-1, 2), omv)
        assert np.array_equal(sad[p].reshape(-1), osad)


def test_cif_many_pairs_multi_macroblock_ctas():
    """R = 16 streamed-frames kernel with more macroblocks than resident CTAs (24 CIF pairs:
    9,504 macroblocks on 2,368 one-warp CTAs), so CTAs alternate pipeline stages: every
    macroblock equals the oracle."""
    W, H, R, P = 352, 288, 16, 24
    fr = sp_inputs.me_sequence(P + 1, W, H, R, seed=91)
    mv, sad = sp.me_search(fr, W, H, R)
    mv, sad = mv.numpy(), sad.numpy().view(np.uint32)
    for p in range(P):
        omv, osad, _ = oracle.me_search(fr[p], fr[p + 1], W, H, R)
        assert np.array_equal(mv[p].reshape(-1, 2), omv), p
        assert np.array_equal(sad[p].reshape(-1), osad), p


def test_1080p_batch_equals_device_path_and_oracle_samples():
    W, H, R = 1920, 1080, 32
    fr = sp_inputs.me_sequence(9, W, H, R)
    ctx = sp.MESearchHost(9, W, H, fr.shape[2], R)
    h = torch.from_numpy(fr).pin_memory()
    for _ in range(2):  # reuse of the staging buffers and flags
        mv, sad = ctx.run(h)
        torch.cuda.synchronize()
        dmv, dsad = _device_path(fr, W, H, R)
        assert np.array_equal(mv.numpy(), dmv) and np.array_equal(sad.numpy(), dsad)
    mbs = [(0, 0), (119, 0), (0, 66), (119, 66), (60, 33), (7, 1)]
    for p in (0, 7):
        omv, osad, _ = oracle.me_search(fr[p], fr[p + 1], W, H, R, mbs=[by * (W // 16) + bx for bx, by in mbs])
        for k, (bx, by) in enumerate(mbs):
            assert tuple(mv[p, by, bx].tolist()) == tuple(omv[k].tolist())
            assert int(sad[p, by, bx]) & 0xFFFFFFFF == int(osad[k])


def test_device_outputs_and_caller_copy_stream():
    W, H, R = 352, 288, 32
    fr = sp_inputs.me_sequence(4, W, H, R)
    h = torch.from_numpy(fr).pin_memory()
    dev = torch.empty_like(h, device="cuda")
    ready = torch.empty(3, dtype=torch.int32, device="cuda")
    mv = torch.empty((3, H // 16, W // 16, 2), dtype=torch.int16, device="cuda")
    sad = torch.empty((3, H // 16, W // 16), dtype=torch.int32, device="cuda")
    cs = torch.cuda.Stream()
    sp._check(sp.lib.sp_me_search_host(h.data_ptr(), fr.shape[2], W, H, 4, R, dev.data_ptr(), ready.data_ptr(),
                                       mv.data_ptr(), sad.data_ptr(), torch.cuda.current_stream().cuda_stream,
                                       cs.cuda_stream), "sp_me_search_host")
    torch.cuda.synchronize()
    dmv, dsad = _device_path(fr, W, H, R)
    assert np.array_equal(mv.cpu().numpy(), dmv) and np.array_equal(sad.cpu().numpy(), dsad)
    assert np.array_equal(dev.cpu().numpy(), fr)  # the staged frames are the input


def test_rejects_pageable_and_unsupported_range():
    W, H = 64, 48
    fr = sp_inputs.me_sequence(3, W, H, 16)
    pageable = torch.from_numpy(fr)
    ctx = sp.MESearchHost(3, W, H, fr.shape[2], 16)
    with pytest.raises(sp.SPError):
        sp._check(sp.lib.sp_me_search_host(pageable.data_ptr(), fr.shape[2], W, H, 3, 16, ctx.frames_dev.data_ptr(),
                                           ctx.ready.data_ptr(), ctx.mv.data_ptr(), ctx.sad.data_ptr(), None, None),
                  "sp_me_search_host")
    h = pageable.pin_memory()
    with pytest.raises(sp.SPError):
        sp._check(sp.lib.sp_me_search_host(h.data_ptr(), fr.shape[2], W, H, 3, 8, ctx.frames_dev.data_ptr(),
                                           ctx.ready.data_ptr(), ctx.mv.data_ptr(), ctx.sad.data_ptr(), None, None),
                  "sp_me_search_host")
    # a single frame holds no pair: nothing to do
    sp._check(sp.lib.sp_me_search_host(h.data_ptr(), fr.shape[2], W, H, 1, 16, ctx.frames_dev.data_ptr(),
                                       ctx.ready.data_ptr(), ctx.mv.data_ptr(), ctx.sad.data_ptr(), None, None),
              "sp_me_search_host")
