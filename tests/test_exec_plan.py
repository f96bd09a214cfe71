"""Host-side parity of the executor's compiled data movement (sp_exec_block with dry_run:
the C++ compile without a launch) against the oracle's sets: the paper's default movement
(Figure 1's printed move-in / move-out code) and the §3.1.4 dataflow
movement.  No GPU needed."""
import numpy as np
import pytest
import torch

import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
from oracle.exec import movement_sets
from tests import exec_programs as X


def _cases():
    blk, bodies, boxes, _ = X.figure1()
    yield "figure1", blk, bodies, boxes, None, [(200, 200), (200, 200)], None
    yield "figure1_tempA", blk, bodies, boxes, None, [(200, 200), (200, 200)], [0, 1]
    blk, bodies, boxes, tiles = X.matvec(20, 28, 8)
    yield "matvec", blk, bodies, boxes, tiles, [(20,), (20, 28), (28,)], None
    blk, bodies, boxes, tiles = X.stencil(23, 31, 8)
    yield "stencil", blk, bodies, boxes, tiles, [(23, 31), (23, 31)], None
    blk, bodies, boxes = X.pipeline(40)
    yield "pipeline", blk, bodies, boxes, None, [(40,), (40,), (40,)], [1, 0, 1]
    blk, bodies, boxes = X.chain(30)
    yield "chain", blk, bodies, boxes, None, [(30,)], None


@pytest.mark.parametrize("case", list(_cases()), ids=lambda c: c[0])
def test_dataflow_move_counts_equal_oracle(case):
    name, blk, bodies, boxes, tiles, shapes, live = case
    arrays = [torch.zeros(s) for s in shapes]
    st = sp.exec_block(blk, bodies, arrays, tile_params=tiles, movement=sp.MOVE_DATAFLOW, live_out=live, dry_run=True)
    want = movement_sets(blk, bodies, shapes, tile_params=tiles, boxes=boxes, live_out=live)
    got = st["move_counts"]
    for t in range(len(want)):
        for a in range(len(shapes)):
            assert tuple(got[t, a]) == (len(want[t][a][0]), len(want[t][a][1])), (name, t, a)
    assert st["moved_in"] == got[:, :, 0].sum() and st["moved_out"] == got[:, :, 1].sum()


def test_default_movement_is_figure1_printed_code():
    blk, bodies, boxes, printed = X.figure1()
    st = sp.exec_block(blk, bodies, [torch.zeros(200, 200), torch.zeros(200, 200)], dry_run=True)
    # Figure 1 move-in A: rows 10-14 x cols 11-20 (50) + the i in 20..28 triangle (25); B: 9 x 10
    assert st["move_counts"][0].tolist() == [[75, 25], [90, 70]]
    assert st["smem_bytes"] == 4 * (19 * 10 + 19 * 24)


def test_dataflow_never_moves_more_than_default():
    for name, blk, bodies, boxes, tiles, shapes, live in _cases():
        arrays = [torch.zeros(s) for s in shapes]
        a = sp.exec_block(blk, bodies, arrays, tile_params=tiles, hoist=False, dry_run=True)["move_counts"]
        b = sp.exec_block(blk, bodies, arrays, tile_params=tiles, movement=sp.MOVE_DATAFLOW, live_out=live,
                          dry_run=True)["move_counts"]
        assert np.all(b <= a), name


def test_compressed_buffers_dry_run():
    """§3.1.2 compression in the executor's compile (reading R-P8): the diagonal program's
    A buffer is 1-D (t + 1 elements per tile: A[i][i] and A[i+1][i+1] for i in the tile)
    instead of the (t + 1)^2 box; moves are unchanged (the same elements cross)."""
    n, t = 40, 8
    blk, bodies, boxes, tiles = X.diagonal(n, t)
    arrays = [torch.zeros(n), torch.zeros(n, n)]
    full = sp.exec_block(blk, bodies, arrays, tile_params=tiles, dry_run=True)
    comp = sp.exec_block(blk, bodies, arrays, tile_params=tiles, dry_run=True, compress=True)
    assert full["smem_bytes"] == 4 * (t + (t + 1) * (t + 1))
    assert comp["smem_bytes"] == 4 * (t + (t + 1))
    assert comp["moved_in"] == full["moved_in"] and comp["moved_out"] == full["moved_out"]
    assert np.array_equal(comp["move_counts"], full["move_counts"])
