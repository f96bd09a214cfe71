"""Multi-process (world_size 2 and 3, gloo on CPU) test of the multi-GPU decomposition:
the slab / halo protocol of sp_jacobi1d_timetiled_dist (csrc/comm.cpp: per pass, send the
first H owned cells left and the last H owned cells right, receive the halos, run the pass
on [x_begin - H, x_end + H)) and the macroblock-row sharding of ME (partition.py), with the
oracle as the per-rank compute.  Gathered results must equal the single-process oracle."""
import os
import socket

import numpy as np
import pytest
import torch.multiprocessing as mp

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, n, steps, tt, W, H, R, pairs, out_dir):
    import sys
    sys.path.insert(0, ROOT)
    import torch
    import torch.distributed as dist

    import oracle
    import sp_inputs
    from paper_conf_ppopp_baskaranbkrrs08_b200 import partition as part

    dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=rank, world_size=world)
    Hh = (tt + 3) & ~3
    # ---- Jacobi: slab + halos, regenerated locally (counter-based generator)
    xb, nl = part.jacobi_slabs(n, world, Hh)[rank]
    buf = np.zeros(nl + 2 * Hh, dtype=np.float32)
    lo, hi = max(0, xb - Hh), min(n, xb + nl + Hh)
    buf[lo - (xb - Hh): hi - (xb - Hh)] = sp_inputs.jacobi_input(hi - lo, seed=7, begin=lo)
    left = rank - 1 if xb > 0 else -1
    right = rank + 1 if xb + nl < n else -1
    done = 0
    while done < steps:
        h = min(tt, steps - done)
        reqs = []
        if left >= 0:
            reqs.append(dist.isend(torch.from_numpy(buf[Hh:2 * Hh].copy()), left))
        if right >= 0:
            reqs.append(dist.isend(torch.from_numpy(buf[nl:nl + Hh].copy()), right))
        if left >= 0:
            t = torch.empty(Hh)
            dist.recv(t, left)
            buf[0:Hh] = t.numpy()
        if right >= 0:
            t = torch.empty(Hh)
            dist.recv(t, right)
            buf[Hh + nl:2 * Hh + nl] = t.numpy()
        for r_ in reqs:
            r_.wait()
        # the pass: cells outside [0, n) are not real; hand the oracle only the real window
        wlo, whi = max(0, xb - Hh), min(n, xb + nl + Hh)
        win = buf[wlo - (xb - Hh): whi - (xb - Hh)]
        buf[wlo - (xb - Hh): whi - (xb - Hh)] = oracle.jacobi1d_window(win, wlo, n, h)
        done += h
    def gather_rows(x):  # all_gather of variable-length row blocks (gloo needs equal sizes)
        sizes = [torch.zeros(1, dtype=torch.int64) for _ in range(world)]
        dist.all_gather(sizes, torch.tensor([x.shape[0]]))
        m = max(int(s_.item()) for s_ in sizes)
        pad = torch.zeros((m,) + tuple(x.shape[1:]), dtype=x.dtype)
        pad[: x.shape[0]] = x
        out = [torch.zeros_like(pad) for _ in range(world)]
        dist.all_gather(out, pad)
        return torch.cat([o[: int(s_.item())] for o, s_ in zip(out, sizes)])

    jac = gather_rows(torch.from_numpy(buf[Hh:Hh + nl].copy()))
    if rank == 0:
        np.save(os.path.join(out_dir, "jac.npy"), jac.numpy())
    # ---- ME: contiguous (pair, MB row) ranges balanced by valid candidates, R-row halo bands
    mby, mbx = H // 16, W // 16
    b, e = part.me_row_ranges(pairs, H, R, world)[rank]
    res = []
    for (p, r0, r1) in part.split_flat_range(b, e, mby):
        row0, row1 = part.me_band_rows(r0, r1, H, R)
        ref = np.zeros((H, W), np.uint8)
        cur = np.zeros((H, W), np.uint8)
        ref[row0:row1] = sp_inputs.me_frame(p, W, H, R, seed=5, row_begin=row0, row_end=row1)
        cur[row0:row1] = sp_inputs.me_frame(p + 1, W, H, R, seed=5, row_begin=row0, row_end=row1)
        mbs = np.arange(r0 * mbx, r1 * mbx, dtype=np.int32)
        mv, sad, _ = oracle.me_search(ref, cur, W, H, R, mbs=mbs)
        res.append(np.concatenate([mv.astype(np.int64), sad.astype(np.int64)[:, None]], axis=1))
    me = gather_rows(torch.from_numpy(np.concatenate(res) if res else np.zeros((0, 3), np.int64)))
    if rank == 0:
        np.save(os.path.join(out_dir, "me.npy"), me.numpy())
    dist.destroy_process_group()


@pytest.mark.parametrize("world", [2, 3])
def test_partitioned_equals_single_process(world, tmp_path):
    import oracle
    import sp_inputs
    n, steps, tt = 5003, 37, 8
    W, H, R, pairs = 96, 80, 8, 3
    mp.spawn(_worker, args=(world, _free_port(), n, steps, tt, W, H, R, pairs, str(tmp_path)), nprocs=world, join=True)
    jac = np.load(tmp_path / "jac.npy")
    want = oracle.jacobi1d(sp_inputs.jacobi_input(n, seed=7), steps)
    assert np.array_equal(jac.view(np.uint32), want.view(np.uint32))
    me = np.load(tmp_path / "me.npy")
    fr = sp_inputs.me_sequence(pairs + 1, W, H, R, seed=5)
    rows = []
    for p in range(pairs):
        mv, sad, _ = oracle.me_search(fr[p], fr[p + 1], W, H, R)
        rows.append(np.concatenate([mv.astype(np.int64), sad.astype(np.int64)[:, None]], axis=1))
    assert np.array_equal(me, np.concatenate(rows))


def test_partition_helpers():
    from paper_conf_ppopp_baskaranbkrrs08_b200 import partition as part
    sl = part.jacobi_slabs(1 << 20, 8, 32)
    assert sl[0][0] == 0 and sum(nl for _, nl in sl) == 1 << 20 and all(xb % 4 == 0 for xb, _ in sl)
    rr = part.me_row_ranges(64, 1080, 32, 8)
    assert rr[0][0] == 0 and rr[-1][1] == 64 * 67 and all(a <= b for a, b in rr)
    w = [part.me_valid_dy(16 * (k % 67), 1080, 32) for k in range(64 * 67)]
    loads = [sum(w[a:b]) for a, b in rr]
    assert max(loads) / min(loads) < 1.01
    assert part.me_band_rows(0, 5, 1080, 32) == (0, 112)
    assert part.split_flat_range(60, 140, 67) == [(0, 60, 67), (1, 0, 67), (2, 0, 6)]
