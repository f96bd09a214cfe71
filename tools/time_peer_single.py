"""Device time of the multi-GPU Jacobi entry points on ONE rank (no neighbours: the halo
protocol is idle) at J3, next to the single-GPU persistent call — the per-GPU cost a rank of
the N > 1 bench pays before any waiting (development aid):  python tools/time_peer_single.py"""
import os
import sys

import torch
import torch.distributed as dist

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402


def ev_time(fn, reps=5, warm=2):
    for _ in range(warm):
        fn()
    torch.cuda.synchronize()
    ts = []
    for _ in range(reps):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        fn()
        b.record()
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b))
    return min(ts)


def main():
    os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
    os.environ.setdefault("MASTER_PORT", "29571")
    dist.init_process_group("gloo", rank=0, world_size=1)
    n, T, tt = 1 << 26, 1024, 64
    a0 = torch.from_numpy(sp_inputs.jacobi_input(n)).cuda()
    a, w = a0.clone(), torch.empty_like(a0)
    print(f"sp_jacobi1d_timetiled_fused (single GPU): {ev_time(lambda: sp.jacobi1d_timetiled_fused(a, T, tt, 0, work=w)):.3f} ms")
    for fused in (False, True):
        slab = sp.PeerSlab(n, 0, n, tt, fused=fused)
        slab.a[slab.H:slab.H + n] = a0
        name = "sp_jacobi1d_timetiled_peer_fused" if fused else "sp_jacobi1d_timetiled_peer (per pass)"
        print(f"{name}: {ev_time(lambda: slab.run(T)):.3f} ms")
        slab.close()
    dist.destroy_process_group()


if __name__ == "__main__":
    main()
