"""GPU parity of the staged-tile executor (sp_exec_block) against the
oracle (oracle/exec.py: the untransformed program on the global arrays).  fp32 with one
IEEE operation per postfix instruction on both sides: results must be bit-identical."""
import numpy as np
import pytest
import torch

import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
from oracle.exec import run_block
from tests import exec_programs as X

pytestmark = pytest.mark.gpu


def _gpu(arrays, *args, **kw):
    d = [torch.from_numpy(a.copy()).cuda() for a in arrays]
    stats = sp.exec_block(*args[:2], d, *args[2:], **kw)
    torch.cuda.synchronize()
    return [t.cpu().numpy() for t in d], stats


def test_figure1_buffers_moves_and_result():
    blk, bodies, boxes, printed = X.figure1()
    rng = np.random.default_rng(0)
    A = rng.standard_normal((200, 200)).astype(np.float32)
    B = rng.standard_normal((200, 200)).astype(np.float32)
    want = run_block(blk, bodies, [A, B], boxes=boxes)
    got, st = _gpu([A, B], blk, bodies)
    assert np.array_equal(got[0], want[0]) and np.array_equal(got[1], want[1])
    # Figure 1's printed storage LA[19][10], LB[19][24] and its move-in /
    # move-out code: A in 50 + 25 = 75 cells, B in 9 x 10 = 90; A out 5 x 5 = 25, B out 5 x 14 = 70
    assert st["smem_bytes"] == 4 * (19 * 10 + 19 * 24)
    assert st["moved_in"] == 75 + 90 and st["moved_out"] == 25 + 70
    assert st["instances"] == 25 + 250


@pytest.mark.parametrize("hoist", [True, False])
def test_matvec_tiles_and_hoisting(hoist):
    n, m, t = 70, 100, 16
    blk, bodies, boxes, tiles = X.matvec(n, m, t)
    rng = np.random.default_rng(1)
    arrs = [rng.standard_normal(n).astype(np.float32), rng.standard_normal((n, m)).astype(np.float32),
            rng.standard_normal(m).astype(np.float32)]
    want = run_block(blk, bodies, arrs, tile_params=tiles, boxes=boxes)
    nJ = (m + t - 1) // t
    got, st = _gpu(arrs, blk, bodies, tile_params=tiles, tiles_per_cta=nJ, hoist=hoist)
    assert np.array_equal(got[0], want[0])
    assert st["ctas"] == (n + t - 1) // t
    assert st["max_levels"] == t  # the j-chain of each y[i]; the i's run in parallel
    if hoist:  # y moved in once and out once per CTA instead of once per tile
        assert st["moves_hoisted"] == 2 * (nJ - 1) * n
    else:
        assert st["moves_hoisted"] == 0


@pytest.mark.parametrize("reuse_filter", [False, True])
def test_stencil_independent_tiles(reuse_filter):
    n, m, t = 67, 93, 16
    blk, bodies, boxes, tiles = X.stencil(n, m, t)
    rng = np.random.default_rng(2)
    arrs = [rng.standard_normal((n, m)).astype(np.float32), np.zeros((n, m), np.float32)]
    want = run_block(blk, bodies, arrs, tile_params=tiles, boxes=boxes)
    got, st = _gpu(arrs, blk, bodies, tile_params=tiles, tiles_per_cta=1, reuse_filter=reuse_filter)
    assert np.array_equal(got[1], want[1]) and np.array_equal(got[0], arrs[0])
    assert st["max_levels"] == 1 and st["ctas"] == len(tiles)
    if reuse_filter:  # B's single write reference has no reuse (Alg. 1): written straight to global
        assert st["moved_out"] == 0


@pytest.mark.parametrize("war", [False, True])
def test_dependence_levels(war):
    n = 300
    blk, bodies, boxes = X.chain(n, war=war)
    a = np.random.default_rng(3).standard_normal(n).astype(np.float32)
    want = run_block(blk, bodies, [a], boxes=boxes)
    got, st = _gpu([a], blk, bodies)
    assert np.array_equal(got[0], want[0])
    assert st["max_levels"] == n - 1


def test_rejects_out_of_bounds_access():
    blk, bodies, boxes = X.chain(10)
    a = torch.zeros(5, device="cuda")  # the block touches a[0..9]
    with pytest.raises(sp.SPError):
        sp.exec_block(blk, bodies, [a])


def test_dataflow_movement_results():
    """§3.1.4 movement changes what is moved, never the live-out results."""
    blk, bodies, boxes, _ = X.figure1()
    rng = np.random.default_rng(5)
    A = rng.standard_normal((200, 200)).astype(np.float32)
    B = rng.standard_normal((200, 200)).astype(np.float32)
    want = run_block(blk, bodies, [A, B], boxes=boxes)
    got, st = _gpu([A, B], blk, bodies, movement=sp.MOVE_DATAFLOW)
    assert np.array_equal(got[0], want[0]) and np.array_equal(got[1], want[1])
    assert st["moved_in"] == 70 + 90 and st["moved_out"] == 25 + 70
    n, m, t = 70, 100, 16
    blk, bodies, boxes, tiles = X.matvec(n, m, t)
    arrs = [rng.standard_normal(n).astype(np.float32), rng.standard_normal((n, m)).astype(np.float32),
            rng.standard_normal(m).astype(np.float32)]
    want = run_block(blk, bodies, arrs, tile_params=tiles, boxes=boxes)
    got, st = _gpu(arrs, blk, bodies, tile_params=tiles, tiles_per_cta=(m + t - 1) // t, movement=sp.MOVE_DATAFLOW)
    assert np.array_equal(got[0], want[0])


def test_dataflow_temporary_stays_on_chip():
    n = 1000
    blk, bodies, boxes = X.pipeline(n)
    rng = np.random.default_rng(6)
    arrs = [rng.standard_normal(n).astype(np.float32), np.full(n, 7.0, np.float32), np.zeros(n, np.float32)]
    want = run_block(blk, bodies, arrs, boxes=boxes)
    got, st = _gpu(arrs, blk, bodies, movement=sp.MOVE_DATAFLOW, live_out=[1, 0, 1])
    assert np.array_equal(got[2], want[2])  # b = a * 2 + 1
    assert np.all(got[1] == 7.0)            # t was produced and consumed in shared memory only
    assert st["moved_in"] == n and st["moved_out"] == n


@pytest.mark.parametrize("compress", [False, True])
def test_diagonal_compressed_buffers(compress):
    """§3.1.2 dimension compression (reading R-P8): the A buffer of the diagonal program is
    staged 1-D; the result is bit-identical to the untransformed program either way."""
    n, t = 70, 16
    blk, bodies, boxes, tiles = X.diagonal(n, t)
    rng = np.random.default_rng(5)
    arrs = [rng.standard_normal(n).astype(np.float32), rng.standard_normal((n, n)).astype(np.float32)]
    want = run_block(blk, bodies, arrs, tile_params=tiles, boxes=boxes)
    got, st = _gpu(arrs, blk, bodies, tile_params=tiles, compress=compress)
    assert np.array_equal(got[0], want[0]) and np.array_equal(got[1], want[1])
    assert st["smem_bytes"] == 4 * (t + ((t + 1) if compress else (t + 1) * (t + 1)))
