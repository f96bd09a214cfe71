"""the paper's tile-size search (§4.3) with libsp sp_tile_search.

Two uses (host only, prints JSON lines):
1. The paper's own settings (8800 GTX: P_low = 32 threads .. 256, M_up = 16 KB / blocks per
   multiprocessor) for the ME nest of Fig. 2 and the Jacobi
   band, sweeping the unstated cost constants S (sync per process) and L (per element):
   which (S, L) ratios reproduce the paper's optima, ME (32,16,16,16) and Jacobi
   (space 256, time 32)?  — "parity unpinned" (S, L are not in the paper).
2. B200 settings (P = 128-256 threads, M_up = the CTA's shared-memory budget), constants from
   the measured microarchitecture (CTA barrier ~ 40 cycles; moving one 4-byte element by
   TMA at ~22 B/clk/SM -> L ~ 0.2 cycles per element per SM, i.e. 0.2*P per process).
    python tools/n2_tile_search.py
"""
import json
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


def main():
    # ---- 1. paper settings ---------------------------------------------------------------
    # ME: problem 8192 x 8192 search positions (Figs. 4/6 "64M"), WS = 16; 32 blocks share 16
    # multiprocessors -> 2 blocks per MP -> M_up = 8 KB = 8192 one-byte elements; P = 256.
    for ratio in [0.01, 0.1, 1, 10, 100, 1000]:
        r = sp.tile_search([8192, 8192, 16, 16], ME_REFS, [POW2, POW2, [4, 8, 16], [4, 8, 16]], mup_elems=8192,
                           procs=256, sync_cost=ratio, elem_cost=1.0)
        print(json.dumps({"exp": "paper_me", "S_over_L": ratio, "tile_ijkl": r["tile"], "cost": r["cost"],
                          "local_elems": r["local_elems"], "paper_optimum": [32, 16, 16, 16]}))
    # Jacobi large N: 128 blocks, 64 threads, M_up = 2^11 bytes = 2^9 words
    for ratio in [0.01, 0.1, 1, 10, 100, 1000]:
        r = sp.tile_search([4096, 512 * 1024], JAC_REFS, [[8, 16, 32, 64, 128], [32, 64, 128, 256, 512]],
                           mup_elems=512, procs=64, sync_cost=ratio, elem_cost=1.0)
        print(json.dumps({"exp": "paper_jacobi", "S_over_L": ratio, "tile_time_space": r["tile"], "cost": r["cost"],
                          "local_elems": r["local_elems"], "paper_optimum": [32, 256]}))
    # ---- 2. B200 settings ------------------------------------------------------------------
    P = 128
    S = 40.0          # cycles per CTA barrier (B300_MICROARCH: BAR ~ 20-50 cycles)
    L = 0.18 * P      # cycles per element per process: 4 B elements at ~22 B/clk/SM by TMA
    r = sp.tile_search([8192, 8192, 16, 16], ME_REFS, [POW2 + [128], POW2 + [128], [16], [16]],
                       mup_elems=48 * 1024, procs=P, sync_cost=S, elem_cost=L)
    print(json.dumps({"exp": "b200_me", "P": P, "S": S, "L": L, "mup_bytes": 48 * 1024, "tile_ijkl": r["tile"],
                      "cost": r["cost"], "local_elems": r["local_elems"]}))
    r = sp.tile_search([1024, 1 << 26], JAC_REFS, [[8, 16, 24, 32, 48, 64], [256, 512, 1024, 2048, 4096]],
                       mup_elems=10 * 1024, procs=P, sync_cost=S, elem_cost=L)
    print(json.dumps({"exp": "b200_jacobi", "P": P, "S": S, "L": L, "mup_words": 10 * 1024,
                      "tile_time_space": r["tile"], "cost": r["cost"], "local_elems": r["local_elems"]}))


if __name__ == "__main__":
    main()
