"""Oracle for the staged-tile executor (sp_exec_block).

TEST INFRASTRUCTURE ONLY — see oracle/__init__.py.  Shares no code with the product
(paper_conf_ppopp_baskaranbkrrs08_b200/csrc/exec.cu); reuses only this package's own
brute-force domain enumeration (oracle/planner.py).

What the executor must compute is the ORIGINAL program's result: the staging (local
buffers, local access functions, move-in / move-out, hoisting; §4.2) is a
transformation that must not change it.  So the oracle runs the block untransformed on
the global arrays:

1. per tile (sequentially, in tile order), each statement's domain is enumerated by
   brute force over the caller's enumeration box;
2. every instance gets its original-order key, the 2d+1 schedule
   (beta_0, i_0, beta_1, ..., i_{d-1}, beta_d) of its statement's textual positions, and
   the instances run in lexicographic key order (statement order within equal keys);
3. an instance evaluates its statement's postfix right-hand side in numpy float32 (one
   IEEE operation per ADD / SUB / MUL, round to nearest) with loads straight from the
   global arrays through the original access functions F . (i, p, 1), and
   stores to its write reference.
"""
from __future__ import annotations

import numpy as np

from .planner import enumerate_domain

LOAD, CONST, ADD, SUB, MUL = 0, 1, 2, 3, 4


def _subscript(ref: dict, x, params) -> tuple:
    v = list(x) + list(params) + [1]
    return tuple(int(sum(int(a) * int(b) for a, b in zip(row, v))) for row in ref["rows"])


def run_block(block: dict, bodies: list, arrays: list, tile_params=None, boxes=None) -> list:
    """Run the block on copies of `arrays` (numpy float32) once per tile; return the arrays.

    bodies[s] = {"write_ref": r, "ops": [(op, arg), ...], "beta": [...]} with
    op in LOAD (arg = ref index), CONST (arg = value), ADD, SUB, MUL.
    boxes[s] = enumeration box of statement s (list of (lo, hi) per loop), or a callable
    params -> box."""
    out = [np.array(a, dtype=np.float32, copy=True) for a in arrays]
    tiles = tile_params if tile_params is not None else [block.get("params", [])]
    for params in tiles:
        params = [int(p) for p in params]
        insts = []
        for s, stmt in enumerate(block["stmts"]):
            box = boxes[s](params) if callable(boxes[s]) else boxes[s]
            pts = enumerate_domain(stmt, params, box)
            beta = bodies[s]["beta"]
            for x in pts:
                key = []
                for k in range(stmt["depth"]):
                    key += [int(beta[k]), int(x[k])]
                key.append(int(beta[stmt["depth"]]))
                insts.append((key, s, tuple(int(v) for v in x)))
        insts.sort(key=lambda t: (t[0], t[1]))
        for _, s, x in insts:
            body = bodies[s]
            stack = []
            for op, arg in body["ops"]:
                if op == LOAD:
                    ref = block["refs"][arg]
                    stack.append(out[ref["array"]][_subscript(ref, x, params)])
                elif op == CONST:
                    stack.append(np.float32(arg))
                else:
                    b, a = stack.pop(), stack.pop()
                    with np.errstate(over="ignore", invalid="ignore"):
                        stack.append(np.float32(a + b) if op == ADD else np.float32(a - b) if op == SUB
                                     else np.float32(a * b))
            ref = block["refs"][body["write_ref"]]
            out[ref["array"]][_subscript(ref, x, params)] = stack[0]
    return out


def movement_sets(block: dict, bodies: list, shapes: list, tile_params=None, boxes=None, live_out=None):
    """§3.1.4 by direct simulation, with the tiles in order as the program.

    Returns [tile][array] -> (move_in set, move_out set) of element coordinates:
    * move in  = elements the tile reads before it writes them itself (the value comes
      from an earlier tile or from the input);
    * move out = elements the tile writes such that the next later tile touching the
      element reads it before writing it, or no later tile writes it and the array is
      live-out (default: every array live-out)."""
    tiles = tile_params if tile_params is not None else [block.get("params", [])]
    n_arrays = len(shapes)
    live = [True] * n_arrays if live_out is None else [bool(v) for v in live_out]
    trace = []  # per tile: ordered list of (reads [(array, coords)], write (array, coords))
    for params in tiles:
        params = [int(p) for p in params]
        insts = []
        for s, stmt in enumerate(block["stmts"]):
            box = boxes[s](params) if callable(boxes[s]) else boxes[s]
            beta = bodies[s]["beta"]
            for x in enumerate_domain(stmt, params, box):
                key = []
                for k in range(stmt["depth"]):
                    key += [int(beta[k]), int(x[k])]
                key.append(int(beta[stmt["depth"]]))
                insts.append((key, s, tuple(int(v) for v in x)))
        insts.sort(key=lambda t: (t[0], t[1]))
        ops = []
        for _, s, x in insts:
            reads = [(block["refs"][a]["array"], _subscript(block["refs"][a], x, params))
                     for op, a in bodies[s]["ops"] if op == LOAD]
            w = block["refs"][bodies[s]["write_ref"]]
            ops.append((reads, (w["array"], _subscript(w, x, params))))
        trace.append(ops)

    def first_access(t, e):  # 'r' (read before any write), 'w', or None
        for reads, w in trace[t]:
            if e in reads:
                return "r"
            if w == e:
                return "w"
        return None

    out = []
    for t, ops in enumerate(trace):
        written, mi, mo = set(), [set() for _ in range(n_arrays)], [set() for _ in range(n_arrays)]
        for reads, w in ops:
            for e in reads:
                if e not in written:
                    mi[e[0]].add(e[1])
            written.add(w)
        for e in written:
            need = live[e[0]]
            for t2 in range(t + 1, len(trace)):
                f = first_access(t2, e)
                if f is not None:
                    need = f == "r"
                    break
            if need:
                mo[e[0]].add(e[1])
        out.append([(mi[a], mo[a]) for a in range(n_arrays)])
    return out
