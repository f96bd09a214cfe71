"""Fused peer-memory halo exchange (sp_jacobi1d_timetiled_peer, and its persistent form
sp_jacobi1d_timetiled_peer_fused) across processes.

The box has one GPU, so the ranks are processes sharing it: buffers and flags are exported
with CUDA IPC and the pass kernels store halos straight into the neighbours' buffers — the
same code path as NVLink peer stores between GPUs.  Two calls per run exercise the
call-boundary handshake.  Results must equal the single-process oracle bit for bit."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.multiprocessing as mp

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, n, steps_list, tt, out_dir, fused=False, space_tile=256):
    import sys
    sys.path.insert(0, ROOT)
    import torch
    import torch.distributed as dist

    import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
    import sp_inputs
    from paper_conf_ppopp_baskaranbkrrs08_b200.partition import jacobi_slabs

    # one GPU per rank when the box has several (NVLink peer memory between devices), else
    # every rank shares GPU 0 (CUDA IPC between processes on one device: the same code path)
    torch.cuda.set_device(rank % torch.cuda.device_count())
    dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=rank, world_size=world)
    H = sp.halo_of(tt)
    xb, nl = jacobi_slabs(n, world, H)[rank]
    slab = sp.PeerSlab(n, xb, nl, tt, space_tile=space_tile, fused=fused)
    slab.a[H:H + nl] = torch.from_numpy(sp_inputs.jacobi_input(nl, seed=31, begin=xb)).cuda()
    torch.cuda.synchronize()
    dist.barrier()
    for st in steps_list:
        slab.run(st)
    torch.cuda.synchronize()
    np.save(os.path.join(out_dir, f"r{rank}.npy"), slab.a[H:H + nl].cpu().numpy())
    slab.close()
    dist.destroy_process_group()


@pytest.mark.timeout(600)
@pytest.mark.parametrize("world", [2, 3])
def test_peer_fused_halo_equals_oracle(world, tmp_path):
    import oracle
    import sp_inputs
    n, tt, steps_list = 12011, 16, [37, 16]
    mp.spawn(_worker, args=(world, _free_port(), n, steps_list, tt, str(tmp_path)), nprocs=world, join=True)
    got = np.concatenate([np.load(tmp_path / f"r{r}.npy") for r in range(world)])
    want = oracle.jacobi1d(sp_inputs.jacobi_input(n, seed=31), sum(steps_list))
    assert np.array_equal(got.view(np.uint32), want.view(np.uint32))


@pytest.mark.timeout(600)
@pytest.mark.parametrize("world,space_tile,n,tt,steps_list", [
    (2, 256, 12011, 16, [37, 16, 5]), (3, 256, 12011, 16, [37, 16, 5]), (2, 8, 12011, 16, [37, 16, 5]),
    # the bench's N > 1 time tile with the persistent in-place geometry (space tile 0)
    (2, 0, 50021, 128, [300, 128, 7]), (3, 0, 50021, 128, [300, 128, 7])])
def test_peer_persistent_halo_equals_oracle(world, space_tile, n, tt, steps_list, tmp_path):
    """sp_jacobi1d_timetiled_peer_fused: every pass of a call in one persistent launch per
    rank, halos pushed by the last edge tile of each side (space tile 8 < halo 16: two edge
    tiles per side).  Three calls exercise the call-boundary handshake."""
    import oracle
    import sp_inputs
    mp.spawn(_worker, args=(world, _free_port(), n, steps_list, tt, str(tmp_path), True, space_tile), nprocs=world,
             join=True)
    got = np.concatenate([np.load(tmp_path / f"r{r}.npy") for r in range(world)])
    want = oracle.jacobi1d(sp_inputs.jacobi_input(n, seed=31), sum(steps_list))
    assert np.array_equal(got.view(np.uint32), want.view(np.uint32))
