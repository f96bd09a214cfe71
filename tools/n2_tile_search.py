"""the paper's tile-size search (§4.3) with libsp sp_tile_search,
its two constants S and L CALIBRATED by B200 microbenchmarks (tools/microbench/n2_calib.cu ->
profiles/r02_n2_calibration.json), and the model's optimum set beside N1's measured optimum.

    python tools/n2_tile_search.py [calibration.json]   -> JSON lines (profiles/r02_n2_tile_search.jsonl)

Model: C = sum_k prod_{i<=r_k} (N_i/t_i) (P S + V_k L / P) over staged arrays (moves in and out),
subject to sum_k M_k(t) <= M_up and prod t_i >= P; V_k, M_k from Alg. 2 on the tile box.
Constants, in SM clock cycles:
  S(P) = barrier(P) / P         synchronisation per process per movement (bar.sync with P threads)
  L(P) = P * 4 B / B_sm          moving one 4-byte (Jacobi) or 1-byte (ME) element, B_sm = bulk-TMA
                                 bytes per clock per SM with the kernels' copies in flight
                                 (HBM-bound when every SM streams)
Measured optima (N1, profiles/r01_jacobi_variant_sweep.txt, r01_n1_ablation.jsonl):
  Jacobi J3: time tile 128, space tile 3328 owned (+ 2 x 128 halo = 3584 cells per warp strip,
             the in-place K = 56 geometry, profiles/r02_jacobi_inplace.txt r3p); the staged
             K = 28 geometry's optimum was time tile 64, space tile 1664 (1792-cell strips)
  ME M4: one macroblock's whole 65 x 65 candidate set x 16 x 16 pixels per CTA iteration.
"""
import json
import os
import sys

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402

ME_REFS = [  # Fig. 2 nest (i, j, k, l), S1 read as SAD[i][j] += |cur[k][l] - ref[i+k][j+l]|
    {"array": 0, "is_write": 0, "rank": 2, "rows": [[1, 0, 1, 0, 0], [0, 1, 0, 1, 0]]},
    {"array": 1, "is_write": 0, "rank": 2, "rows": [[0, 0, 1, 0, 0], [0, 0, 0, 1, 0]]},
    {"array": 2, "is_write": 1, "rank": 2, "rows": [[1, 0, 0, 0, 0], [0, 1, 0, 0, 0]]},
    {"array": 2, "is_write": 0, "rank": 2, "rows": [[1, 0, 0, 0, 0], [0, 1, 0, 0, 0]]},
]
JAC_REFS = [  # (t, i') band after skewing i' = i + t (time tiles are parallelograms):
    # b[i] = f(a[i-1], a[i], a[i+1]) becomes a[i' - t - 1], a[i' - t], a[i' - t + 1] -> b[i' - t]
    {"array": 0, "is_write": 0, "rank": 1, "rows": [[-1, 1, -1]]},
    {"array": 0, "is_write": 0, "rank": 1, "rows": [[-1, 1, 0]]},
    {"array": 0, "is_write": 0, "rank": 1, "rows": [[-1, 1, 1]]},
    {"array": 1, "is_write": 1, "rank": 1, "rows": [[-1, 1, 0]]},
]
POW2 = [1, 2, 4, 8, 16, 32, 64]


def constants(cal, P, elem_bytes, chunk):
    bars = {int(k): v for k, v in cal["barrier_cycles"].items()}
    S = bars[P] / P
    # bulk TMA with the most copies in flight per SM at this chunk size (the kernels keep
    # 16 warps x 1 prefetch in flight: HBM-bound)
    rows = [r for r in cal["tma"] if r["bytes"] == chunk and r["ctas_per_sm"] > 0]
    B = max(r["bytes_per_clk_per_sm"] for r in rows)
    return S, P * elem_bytes / B, B


def main():
    path = sys.argv[1] if len(sys.argv) > 1 else os.path.join("profiles", "r02_n2_calibration.json")
    cal = json.load(open(path))
    out = []
    # ---- Jacobi: the (t, i') band of J3, P = 32 lanes of a warp (the outer process is a warp),
    # M_up = one warp strip (K = 28: 1792 fp32 cells; in place K = 56: 3584)
    P = 32
    S, L, B = constants(cal, P, 4, 7168)
    cand_t = [8, 16, 32, 48, 64, 96, 128]
    cand_s = [256, 512, 1024, 1664, 2048, 4096]
    for mup in (1792, 3584, 4096):
        r = sp.tile_search([1024, 1 << 26], JAC_REFS, [cand_t, cand_s], mup_elems=mup, procs=P, sync_cost=S,
                           elem_cost=L)
        out.append({"exp": "b200_jacobi", "P": P, "S_cycles": round(S, 4), "L_cycles": round(L, 4),
                    "tma_bytes_per_clk_sm": B, "mup_words": mup, "model_tile_time_space": r["tile"],
                    "model_cost_cycles": r["cost"], "local_elems": r["local_elems"],
                    "measured_optimum_time_space": [128, 3328] if mup >= 3584 else [64, 1664],
                    "measured_source": ("profiles/r02_jacobi_inplace.txt r3p (in place K = 56: Tt 64 / 96 / 128)"
                                        if mup >= 3584 else
                                        "profiles/r01_jacobi_variant_sweep.txt (staged K = 28: Tt 32..80)")})
    # model cost of the measured optimum and of its neighbours (same objective, fixed tiles)
    for tt, ss in [(64, 1664), (32, 1664), (128, 1664), (64, 1024), (128, 3328), (64, 3456)]:
        r = sp.tile_search([1024, 1 << 26], JAC_REFS, [[tt], [ss]], mup_elems=0, procs=P, sync_cost=S, elem_cost=L)
        out.append({"exp": "b200_jacobi_cost_at", "tile_time_space": [tt, ss], "model_cost_cycles": r["cost"],
                    "local_elems": r["local_elems"]})
    # ---- ME: Fig. 2 nest over ONE macroblock's search (N_i = N_j = 2R + 1 = 65, WS = 16),
    # P = 128 threads (4 warps per CTA), M_up = the CTA's shared-memory budget (52 KB at 4 CTAs/SM)
    P = 128
    S, L, B = constants(cal, P, 1, 6400)
    r = sp.tile_search([65, 65, 16, 16], ME_REFS, [[8, 16, 32, 65], [8, 16, 32, 65], [4, 8, 16], [4, 8, 16]],
                       mup_elems=52 * 1024, procs=P, sync_cost=S, elem_cost=L)
    out.append({"exp": "b200_me", "P": P, "S_cycles": round(S, 4), "L_cycles": round(L, 4),
                "tma_bytes_per_clk_sm": B, "mup_bytes": 52 * 1024, "model_tile_ijkl": r["tile"],
                "model_cost_cycles": r["cost"], "local_elems": r["local_elems"],
                "measured_optimum_ijkl": [65, 65, 16, 16],
                "measured_source": "round-1 ME design: one macroblock's full candidate set per CTA iteration"})
    for o in out:
        print(json.dumps(o))


if __name__ == "__main__":
    main()
