"""B200 analogues of the paper's experiments.

* Figs. 4/5 + the 8x / 10x claims: staged (scratchpad) kernels vs the
  "GPU w/o scratchpad" kernels (libsp sp_jacobi1d_untiled, sp_me_sad_search_direct) at the
  BASELINE configs J3 / M4 and at the paper's problem-size ranges.
* Fig. 8: Jacobi time vs (time, space) tile at the paper's large sizes.
* Fig. 7: Jacobi time vs number of outer tiles (space tile S) at N = 8k-32k,
  T = 4096 (the paper's "fits in scratchpad" regime).
Device time by CUDA events; prints one JSON object per measurement.
    python tools/n1_ablation.py [quick]
"""
import json
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402


def ev(fn, reps=3, warm=1):
    for _ in range(warm):
        fn()
    torch.cuda.synchronize()
    best = 1e30
    for _ in range(reps):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        fn()
        b.record()
        torch.cuda.synchronize()
        best = min(best, a.elapsed_time(b))
    return best


def emit(**kw):
    print(json.dumps(kw), flush=True)


def jacobi_pair(n, T, tt=32, S=0, untiled=True, per_pass=False):
    """staged time (persistent all-pass launch, the product path), DRAM-only time; with
    per_pass the one-launch-per-time-tile staged path is timed instead of the persistent one"""
    a0 = torch.from_numpy(sp_inputs.jacobi_input(n, seed=2008)).cuda()
    a = a0.clone()
    w = torch.empty_like(a)
    plan = sp.jacobi1d_plan(n, T, tt, S)
    fl = torch.empty(plan["tiles"] + 1 + plan["passes"], dtype=torch.int32, device="cuda")
    if per_pass:
        t_st = ev(lambda: sp.jacobi1d_timetiled(a, T, tt, S, work=w))
    else:
        t_st = ev(lambda: sp.jacobi1d_timetiled_fused(a, T, tt, S, work=w, flags=fl))
    t_un = ev(lambda: sp.jacobi1d_untiled(a, T, work=w)) if untiled else None
    return t_st, t_un


def main():
    quick = len(sys.argv) > 1 and sys.argv[1] == "quick"
    # ---- Figs. 4/5 + speedup claims at the BASELINE configs -------------------------------
    n, T = 1 << 26, 1024
    t_st, t_un = jacobi_pair(n, T, 64)
    t_pp, _ = jacobi_pair(n, T, 64, untiled=False, per_pass=True)
    emit(exp="jacobi_staged_vs_dram_only", n=n, T=T, time_tile=64, staged_ms=t_st, staged_per_pass_ms=t_pp,
         dram_only_ms=t_un, speedup=t_un / t_st, paper_speedup_8800gtx=10.0,
         updates_per_s_staged=(n - 2) * T / (t_st * 1e-3))
    W, H, R = 1920, 1080, 32
    fr = torch.from_numpy(sp_inputs.me_sequence(9 if quick else 65, W, H, R)).cuda()
    t_me = ev(lambda: sp.me_search_sequence(fr, W, H, R))
    t_dir = ev(lambda: sp.me_sad_search_direct(fr[:-1], fr[1:], W, H, R), reps=2)
    emit(exp="me_staged_vs_dram_only", frames=fr.shape[0], W=W, H=H, R=R, staged_ms=t_me, dram_only_ms=t_dir,
         speedup=t_dir / t_me, paper_speedup_8800gtx=8.0)
    # ---- Fig. 5 problem-size range (8k..512k), T = 4096 ------------------------------------
    for n in [8 << 10, 32 << 10, 128 << 10, 512 << 10]:
        t_st, t_un = jacobi_pair(n, 4096)
        t_pp, _ = jacobi_pair(n, 4096, untiled=False, per_pass=True)
        t_res = None
        if n <= sp.jacobi1d_resident_capacity():  # the whole domain in one cluster
            a = torch.from_numpy(sp_inputs.jacobi_input(n, seed=2008)).cuda()
            t_res = ev(lambda: sp.jacobi1d_resident(a, 4096))
        emit(exp="fig5_jacobi_size", n=n, T=4096, staged_ms=t_st, staged_per_pass_ms=t_pp, cluster_resident_ms=t_res,
             dram_only_ms=t_un, speedup=t_un / min(t_st, t_res or t_st))
    # ---- Fig. 8: (time, space) tiles at 64k..512k, T = 4096 --------------------------------
    for n in [64 << 10, 512 << 10]:
        for tt, S in [(32, 64), (32, 128), (16, 256), (32, 256), (64, 256), (32, 1024), (32, 0)]:
            try:
                t_st, _ = jacobi_pair(n, 4096, tt, S, untiled=False)
            except sp.SPError:
                continue
            emit(exp="fig8_jacobi_tiles", n=n, T=4096, time_tile=tt, space_tile=S or
                 sp.jacobi1d_plan(n, 4096, tt, 0)["space_tile"], ms=t_st)
    # ---- Fig. 7: number of outer tiles at N = 8k/16k/32k, T = 4096, time tile 32 -------------
    for n in [8 << 10, 16 << 10, 32 << 10]:
        for S in [64, 128, 256, 512, 1024]:
            try:
                t_st, _ = jacobi_pair(n, 4096, 32, S, untiled=False)
            except sp.SPError:
                continue
            t_pp, _ = jacobi_pair(n, 4096, 32, S, untiled=False, per_pass=True)
            emit(exp="fig7_jacobi_tiles_count", n=n, T=4096, space_tile=S, tiles=-(-n // S), ms=t_st, per_pass_ms=t_pp)
    # ---- staged Jacobi across time tiles at J3 (HBM <-> FP32 cross-over) --------------------
    for tt in [4, 8, 16, 24, 32, 48, 64]:
        t_st, _ = jacobi_pair(1 << 26, 1024, tt, 0, untiled=False)
        emit(exp="j3_time_tile_sweep", time_tile=tt, ms=t_st, gupd_s=((1 << 26) - 2) * 1024 / (t_st * 1e-3) / 1e9,
             hbm_alg_gbs=8.0 * (1 << 26) * (1024 / tt) / (t_st * 1e-3) / 1e9)


if __name__ == "__main__":
    main()
