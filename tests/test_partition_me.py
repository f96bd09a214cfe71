"""Host logic of the sharded ME (partition.py, CPU): the ranges cover the batch's (pair, MB row)
space exactly once, balance the valid-candidate count, and the rows a rank holds
(me_needed_rows) are exactly the frame rows its macroblocks read — checked by brute force over
every macroblock's current block and reference window rows intersected with the frame, and the
candidates' rows (valid candidates only read inside the frame)."""
import itertools

import pytest

from paper_conf_ppopp_baskaranbkrrs08_b200 import partition as P


def _rows_read(pieces, f, H, R):
    rows = set()
    for p, r0, r1 in pieces:
        for by in range(r0, r1):
            y0 = 16 * by
            if p + 1 == f:  # current block rows
                rows.update(range(y0, y0 + 16))
            if p == f:  # rows of the valid candidates' reference blocks
                for dy in range(-R, R + 1):
                    if 0 <= y0 + dy and y0 + dy + 16 <= H:
                        rows.update(range(y0 + dy, y0 + dy + 16))
    return rows


@pytest.mark.parametrize("pairs,H,R,world", [(4, 80, 16, 3), (3, 128, 32, 3), (1, 48, 16, 4), (64, 1080, 32, 8),
                                             (5, 288, 16, 7), (2, 1080, 32, 3)])
def test_ranges_partition_and_balance(pairs, H, R, world):
    rs = P.me_row_ranges(pairs, H, R, world)
    mby = H // 16
    assert rs[0][0] == 0 and rs[-1][1] == pairs * mby
    assert all(a[1] == b[0] for a, b in zip(rs, rs[1:])) and all(b >= a for a, b in rs)
    w = [P.me_valid_dy(16 * (k % mby), H, R) for k in range(pairs * mby)]
    loads = [sum(w[a:b]) for a, b in rs]
    assert max(loads) - min(loads) <= 2 * max(w)  # balanced within two rows' weight


@pytest.mark.parametrize("pairs,H,R,world", [(4, 80, 16, 3), (3, 128, 32, 3), (2, 1080, 32, 3), (5, 288, 16, 7)])
def test_needed_rows_equal_rows_read(pairs, H, R, world):
    mby = H // 16
    for fb, fe in P.me_row_ranges(pairs, H, R, world):
        pieces = P.split_flat_range(fb, fe, mby)
        for f in range(pairs + 1):
            got = P.me_needed_rows(pieces, f, H, R)
            want = _rows_read(pieces, f, H, R)
            rows = set()
            for a, b in got:
                assert a < b and not (rows & set(range(a, b)))
                rows |= set(range(a, b))
            # disjoint bands covering exactly the rows read (nothing more is ever loaded)
            assert rows == want, (fb, fe, f, got)
            assert got == sorted(got)


def test_split_flat_range_pieces():
    assert P.split_flat_range(3, 14, 5) == [(0, 3, 5), (1, 0, 5), (2, 0, 4)]
    assert P.split_flat_range(7, 7, 5) == []
    for b, e in itertools.combinations(range(0, 21), 2):
        pieces = P.split_flat_range(b, e, 5)
        assert sum(r1 - r0 for _, r0, r1 in pieces) == e - b
