"""Program blocks for the staged-tile executor tests (sp_exec_block).

Plain data (domains, references, postfix bodies, enumeration boxes) shared by the oracle
tests (CPU) and the GPU parity tests; no method arithmetic lives here."""
import json
import os

HERE = os.path.dirname(os.path.abspath(__file__))
LOAD, CONST, ADD, SUB, MUL = 0, 1, 2, 3, 4


def figure1():
    """P:L500-508 (Figure 1): A[i][j+1] = A[i+j][j+1]*3;  B[i][j+k] = A[i][k] + B[i+j][k]."""
    g = json.load(open(os.path.join(HERE, "golden", "figure1.json")))
    blk = g["block"]
    bodies = [
        {"write_ref": 0, "beta": [0, 0, 0], "ops": [(LOAD, 1), (CONST, 3.0), (MUL, 0)]},
        {"write_ref": 2, "beta": [0, 0, 1, 0], "ops": [(LOAD, 3), (LOAD, 4), (ADD, 0)]},
    ]
    boxes = [s["box"] for s in blk["stmts"]]
    return blk, bodies, boxes, g["printed"]


def matvec(n, m, t):
    """y[i] = y[i] + A[i][j] * x[j], tiles (I, J) of t x t: i in [tI, tI+t), j in [tJ, tJ+t).
    Parameters (I, J).  The y buffer does not depend on J (a redundant tiling loop, §4.2)."""
    dom = [[1, 0, -t, 0, 0], [-1, 0, t, 0, t - 1], [0, 1, 0, -t, 0], [0, -1, 0, t, t - 1],
           [1, 0, 0, 0, 0], [-1, 0, 0, 0, n - 1], [0, 1, 0, 0, 0], [0, -1, 0, 0, m - 1]]
    blk = {"params": [0, 0], "stmts": [{"depth": 2, "rows": dom}], "refs": [
        {"stmt": 0, "array": 0, "is_write": 1, "rank": 1, "rows": [[1, 0, 0, 0, 0]]},           # y[i]
        {"stmt": 0, "array": 0, "is_write": 0, "rank": 1, "rows": [[1, 0, 0, 0, 0]]},           # y[i]
        {"stmt": 0, "array": 1, "is_write": 0, "rank": 2, "rows": [[1, 0, 0, 0, 0], [0, 1, 0, 0, 0]]},  # A[i][j]
        {"stmt": 0, "array": 2, "is_write": 0, "rank": 1, "rows": [[0, 1, 0, 0, 0]]},           # x[j]
    ]}
    bodies = [{"write_ref": 0, "beta": [0, 0, 0], "ops": [(LOAD, 1), (LOAD, 2), (LOAD, 3), (MUL, 0), (ADD, 0)]}]
    tiles = [[I, J] for I in range((n + t - 1) // t) for J in range((m + t - 1) // t)]
    boxes = [lambda p: [(t * p[0], t * p[0] + t - 1), (t * p[1], t * p[1] + t - 1)]]
    return blk, bodies, boxes, tiles


def stencil(n, m, t):
    """B[i][j] = (((A[i-1][j] + A[i+1][j]) + A[i][j-1]) + A[i][j+1]) * 0.25 on the interior,
    tiles (I, J) of t x t over i, j in [1, n-2] x [1, m-2]; parameters (I, J)."""
    dom = [[1, 0, -t, 0, -1], [-1, 0, t, 0, t], [0, 1, 0, -t, -1], [0, -1, 0, t, t],
           [1, 0, 0, 0, -1], [-1, 0, 0, 0, n - 2], [0, 1, 0, 0, -1], [0, -1, 0, 0, m - 2]]

    def ref(arr, w, di, dj):
        return {"stmt": 0, "array": arr, "is_write": w, "rank": 2, "rows": [[1, 0, 0, 0, di], [0, 1, 0, 0, dj]]}
    blk = {"params": [0, 0], "stmts": [{"depth": 2, "rows": dom}],
           "refs": [ref(1, 1, 0, 0), ref(0, 0, -1, 0), ref(0, 0, 1, 0), ref(0, 0, 0, -1), ref(0, 0, 0, 1)]}
    bodies = [{"write_ref": 0, "beta": [0, 0, 0], "ops": [(LOAD, 1), (LOAD, 2), (ADD, 0), (LOAD, 3), (ADD, 0),
                                                          (LOAD, 4), (ADD, 0), (CONST, 0.25), (MUL, 0)]}]
    tiles = [[I, J] for I in range((n - 2 + t - 1) // t) for J in range((m - 2 + t - 1) // t)]
    boxes = [lambda p: [(t * p[0] + 1, t * p[0] + t), (t * p[1] + 1, t * p[1] + t)]]
    return blk, bodies, boxes, tiles


def chain(n, war=False):
    """Loop-carried dependences inside one tile.  Flow: a[i] = a[i-1] + a[i] (i = 1..n-1);
    anti (war=True): a[i] = a[i+1] * 2 (i = 0..n-2, each a[i+1] read before it is overwritten)."""
    if war:
        dom = [[1, 0], [-1, n - 2]]
        refs = [{"stmt": 0, "array": 0, "is_write": 1, "rank": 1, "rows": [[1, 0]]},
                {"stmt": 0, "array": 0, "is_write": 0, "rank": 1, "rows": [[1, 1]]}]
        ops = [(LOAD, 1), (CONST, 2.0), (MUL, 0)]
    else:
        dom = [[1, -1], [-1, n - 1]]
        refs = [{"stmt": 0, "array": 0, "is_write": 1, "rank": 1, "rows": [[1, 0]]},
                {"stmt": 0, "array": 0, "is_write": 0, "rank": 1, "rows": [[1, -1]]},
                {"stmt": 0, "array": 0, "is_write": 0, "rank": 1, "rows": [[1, 0]]}]
        ops = [(LOAD, 1), (LOAD, 2), (ADD, 0)]
    blk = {"params": [], "stmts": [{"depth": 1, "rows": dom}], "refs": refs}
    return blk, [{"write_ref": 0, "beta": [0, 0], "ops": ops}], [[(0, n - 1)]]


def pipeline(n):
    """t[i] = a[i] * 2 (S1); b[i] = t[i] + 1 (S2), both in one loop over i (t is a temporary
    when not live-out).  Arrays: a = 0, t = 1, b = 2."""
    dom = [[1, 0], [-1, n - 1]]

    def r(s, a, w):
        return {"stmt": s, "array": a, "is_write": w, "rank": 1, "rows": [[1, 0]]}
    blk = {"params": [], "stmts": [{"depth": 1, "rows": dom}, {"depth": 1, "rows": dom}],
           "refs": [r(0, 1, 1), r(0, 0, 0), r(1, 2, 1), r(1, 1, 0)]}
    bodies = [{"write_ref": 0, "beta": [0, 0], "ops": [(LOAD, 1), (CONST, 2.0), (MUL, 0)]},
              {"write_ref": 2, "beta": [0, 1], "ops": [(LOAD, 3), (CONST, 1.0), (ADD, 0)]}]
    return blk, bodies, [[(0, n - 1)], [(0, n - 1)]]


def diagonal(n, t):
    """d[i] = A[i][i] * 2 + A[i+1][i+1] (i = 0..n-2), tiles I of t: i in [tI, tI+t).
    Parameter (I).  Both references of A lie on the diagonal, so with §3.1.2 compression
    the staged buffer of A is 1-D (t+1 elements) instead of the (t+1) x (t+1) box."""
    dom = [[1, -t, 0], [-1, t, t - 1], [1, 0, 0], [-1, 0, n - 2]]
    blk = {"params": [0], "stmts": [{"depth": 1, "rows": dom}], "refs": [
        {"stmt": 0, "array": 0, "is_write": 1, "rank": 1, "rows": [[1, 0, 0]]},                   # d[i]
        {"stmt": 0, "array": 1, "is_write": 0, "rank": 2, "rows": [[1, 0, 0], [1, 0, 0]]},        # A[i][i]
        {"stmt": 0, "array": 1, "is_write": 0, "rank": 2, "rows": [[1, 0, 1], [1, 0, 1]]},        # A[i+1][i+1]
    ]}
    bodies = [{"write_ref": 0, "beta": [0, 0], "ops": [(LOAD, 1), (CONST, 2.0), (MUL, 0), (LOAD, 2), (ADD, 0)]}]
    tiles = [[I] for I in range((n - 1 + t - 1) // t)]
    boxes = [lambda p: [(t * p[0], t * p[0] + t - 1)]]
    return blk, bodies, boxes, tiles
