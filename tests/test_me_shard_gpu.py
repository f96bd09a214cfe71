"""Sharded motion estimation (SURVEY §8(e) ME row) on the GPU, against the CPU oracle.

* sp_me_sad_search_range: one flat (pair, MB row) range of a batch, global output indexing,
  frames held from `pair_base` on, rows outside the range's band left as garbage (0xEE) to
  prove only the band (current rows + R-row reference halo) is read — fast (R = 16, 32) and
  generic (other R) kernels.
* sp_me_sad_search_gather (MEShard): ranks are processes sharing the one GPU (CUDA IPC, the
  same code path as NVLink peer stores between GPUs); each rank loads only its band rows,
  searches its range and the kernel stores every result into every rank's outputs.  After the
  call every rank must hold the whole batch, bit-identical to the oracle — including ranges
  that split a pair in the middle (world 3) and a rank with an empty range (world > MB rows).
  Two calls per run exercise the epoch handshake.
* sp_me_sad_search_dist (NCCL broadcast baseline): single rank (NCCL refuses two ranks on one
  device).
Macroblocks are independent FORALL iterations."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.multiprocessing as mp

import oracle
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
import sp_inputs
from paper_conf_ppopp_baskaranbkrrs08_b200 import partition

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _oracle_batch(fr, W, H, R):
    mby, mbx = H // 16, W // 16
    mv = np.zeros((fr.shape[0] - 1, mby, mbx, 2), np.int16)
    sad = np.zeros((fr.shape[0] - 1, mby, mbx), np.uint32)
    for p in range(fr.shape[0] - 1):
        omv, osad, _ = oracle.me_search(fr[p], fr[p + 1], W, H, R)
        mv[p] = omv.reshape(mby, mbx, 2)
        sad[p] = osad.reshape(mby, mbx)
    return mv, sad


@pytest.mark.parametrize("W,H,R,pairs", [(96, 80, 16, 4), (160, 128, 32, 3), (100, 70, 5, 3), (64, 48, 0, 2)])
def test_range_search_equals_oracle(W, H, R, pairs):
    pitch = (W + 15) // 16 * 16
    fr = sp_inputs.me_sequence(pairs + 1, W, H, max(R, 2), seed=11 + R, pitch=pitch)
    omv, osad = _oracle_batch(fr, W, H, R)
    mby = H // 16
    rng = np.random.default_rng(R)
    cuts = sorted(set([0, pairs * mby] + list(rng.integers(0, pairs * mby, size=3))))
    for fb, fe in zip(cuts[:-1], cuts[1:]):
        pieces = partition.split_flat_range(fb, fe, mby)
        p0, p1 = pieces[0][0], pieces[-1][0]
        # frames pair_base .. p1 + 1; everything outside the band rows is garbage
        loc = np.full((p1 - p0 + 2, H, pitch), 0xEE, np.uint8)
        for p, r0, r1 in pieces:
            a, b = partition.me_band_rows(r0, r1, H, R)
            loc[p - p0, a:b] = fr[p, a:b]
            loc[p - p0 + 1, 16 * r0:16 * r1] = fr[p + 1, 16 * r0:16 * r1]
        mv = torch.full((pairs, mby, W // 16, 2), -7, dtype=torch.int16, device="cuda")
        sad = torch.full((pairs, mby, W // 16), -7, dtype=torch.int32, device="cuda")
        sp.me_sad_search_range(torch.from_numpy(loc).cuda(), W, H, R, fb, fe, pair_base=p0, out=(mv, sad))
        torch.cuda.synchronize()
        gmv = mv.cpu().numpy().reshape(pairs * mby, -1, 2)
        gsad = sad.cpu().numpy().view(np.uint32).reshape(pairs * mby, -1)
        assert np.array_equal(gmv[fb:fe], omv.reshape(pairs * mby, -1, 2)[fb:fe])
        assert np.array_equal(gsad[fb:fe], osad.reshape(pairs * mby, -1)[fb:fe])
        # nothing outside the range was written
        assert np.all(np.delete(gmv, np.s_[fb:fe], axis=0) == -7)
        assert np.all(np.delete(gsad.view(np.int32), np.s_[fb:fe], axis=0) == -7)


def _shard_worker(rank, world, port, W, H, R, pairs, out_dir, calls):
    import sys
    sys.path.insert(0, ROOT)
    import torch
    import torch.distributed as dist

    import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
    import sp_inputs

    # one GPU per rank when the box has several (NVLink peer memory between devices), else
    # every rank shares GPU 0 (CUDA IPC between processes on one device: the same code path)
    torch.cuda.set_device(rank % torch.cuda.device_count())
    dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=rank, world_size=world)
    pitch = (W + 15) // 16 * 16
    shard = sp.MEShard(pairs, W, H, R, pitch=pitch)
    for c in range(calls):
        # call c searches sequence c (different frames: stale results cannot pass)
        seq = sp_inputs.me_sequence(pairs + 1, W, H, R, seed=100 + c, pitch=pitch)
        shard.frames.fill_(0xEE)  # rows outside the band stay garbage
        shard.load_frames(lambda f: seq[f])
        mv, sad = shard.run()
        torch.cuda.synchronize()
        np.save(os.path.join(out_dir, f"mv{c}_r{rank}.npy"), mv.cpu().numpy())
        np.save(os.path.join(out_dir, f"sad{c}_r{rank}.npy"), sad.cpu().numpy().view(np.uint32))
        dist.barrier()
    shard.close()
    dist.destroy_process_group()


@pytest.mark.timeout(900)
@pytest.mark.parametrize("world,W,H,R,pairs", [(2, 96, 80, 16, 4), (3, 96, 80, 16, 4), (3, 160, 128, 32, 3),
                                               (2, 160, 128, 32, 1), (4, 64, 48, 16, 1)])
def test_sharded_gather_equals_oracle(world, W, H, R, pairs, tmp_path):
    calls = 2
    mp.spawn(_shard_worker, args=(world, _free_port(), W, H, R, pairs, str(tmp_path), calls), nprocs=world, join=True)
    pitch = (W + 15) // 16 * 16
    for c in range(calls):
        seq = sp_inputs.me_sequence(pairs + 1, W, H, R, seed=100 + c, pitch=pitch)
        omv, osad = _oracle_batch(seq, W, H, R)
        for r in range(world):
            assert np.array_equal(np.load(tmp_path / f"mv{c}_r{r}.npy"), omv), (c, r)
            assert np.array_equal(np.load(tmp_path / f"sad{c}_r{r}.npy"), osad), (c, r)


def test_partition_splits_mid_pair():
    """The world-3 case above really splits a pair between ranks (and world 4 on 3 MB rows
    leaves one rank empty)."""
    rs = partition.me_row_ranges(4, 80, 16, 3)
    assert any(b % 5 != 0 for b, _ in rs[1:])
    rs4 = partition.me_row_ranges(1, 48, 16, 4)
    assert any(b == e for b, e in rs4)


def test_nccl_dist_single_rank():
    """sp_me_sad_search_dist with one rank (the broadcasts are skipped; the range search and
    the argument path are exercised)."""
    W, H, R, pairs = 96, 80, 16, 3
    pitch = 96
    fr = sp_inputs.me_sequence(pairs + 1, W, H, R, seed=5, pitch=pitch)
    omv, osad = _oracle_batch(fr, W, H, R)
    uid = sp.get_unique_id()
    comm = sp.Comm(uid, 1, 0, 0)
    try:
        mby = H // 16
        mv = torch.zeros((pairs, mby, W // 16, 2), dtype=torch.int16, device="cuda")
        sad = torch.zeros((pairs, mby, W // 16), dtype=torch.int32, device="cuda")
        comm.me_sad_search_dist(torch.from_numpy(fr).cuda(), W, H, R, [(0, pairs * mby)], 0, mv, sad)
        torch.cuda.synchronize()
        assert np.array_equal(mv.cpu().numpy(), omv)
        assert np.array_equal(sad.cpu().numpy().view(np.uint32), osad)
    finally:
        comm.destroy()
