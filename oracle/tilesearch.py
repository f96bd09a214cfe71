"""Oracle for the tile-size search objective (§4.3) — TEST INFRASTRUCTURE ONLY.

Exhaustive over the candidate grid, written from the paper's formulation:
  variables t_1..t_m;  constraints 0 < t_i <= N_i, sum_j M_j <= M_up, t_1...t_m >= P;
  objective sum_{k in I} prod_{i<=r_k} (N_i/t_i) (P S + V_in_k L / P)
          + sum_{k in O} prod_{i<=r_k} (N_i/t_i) (P S + V_out_k L / P)
with N_i/t_i read as the number of tiles ceil(N_i/t_i) (integer tile counts, reading R-T1),
M_j, V_in, V_out from the brute-force planner (oracle/planner.py) on the box tile, and r_k
the deepest loop array k's references depend on (movement hoisted above redundant loops,
P:L654-666).
"""
from __future__ import annotations

import itertools

from . import planner as P


def tile_search(extent, refs, candidates, mup_elems=0, procs=32, sync_cost=1.0, elem_cost=1.0):
    m = len(extent)
    arrays = sorted({r["array"] for r in refs})
    rk = {a: -1 for a in arrays}
    for r in refs:
        for row in r["rows"]:
            for l in range(m):
                if row[l] != 0:
                    rk[r["array"]] = max(rk[r["array"]], l)
    best = None
    evaluated = 0
    for t in itertools.product(*candidates):
        prod = 1
        for x in t:
            prod *= x
        if prod < procs:
            continue
        rows = []
        for l in range(m):
            lo = [0] * (m + 1)
            lo[l] = 1
            hi = [0] * (m + 1)
            hi[l] = -1
            hi[m] = t[l] - 1
            rows += [lo, hi]
        blk = {"params": [], "stmts": [{"depth": m, "rows": rows, "box": [[0, x - 1] for x in t]}],
               "refs": [dict(r, stmt=0) for r in refs]}
        plan = P.plan_buffers(blk, mode=P.PER_ARRAY)
        evaluated += 1
        mem = sum(b["size"] for b in plan["buffers"])
        cost = 0.0
        for b in plan["buffers"]:
            moves = 1.0
            for l in range(rk[b["array"]] + 1):
                moves *= float(-(-extent[l] // t[l]))
            if b["in_count"] > 0:
                cost += moves * (procs * sync_cost + b["v_in_ub"] * elem_cost / procs)
            if b["out_count"] > 0:
                cost += moves * (procs * sync_cost + b["v_out_ub"] * elem_cost / procs)
        if mup_elems and mem > mup_elems:
            continue
        if best is None or cost < best["cost"]:
            best = {"tile": list(t), "cost": cost, "local_elems": mem}
    return {"best": best, "evaluated": evaluated}
