"""Pins for the dispatch-semantics reference (Fig. 8b, §2.4, §6.4)."""
import numpy as np
import pytest

from oracle import dispatch_ref as D


@pytest.mark.parametrize("total,quota,chunk", [(20, 4, 1), (12, 2, 1), (8, 2, 1), (1000, 7, 8),
                                               (999, 13, 6), (5, 9, 4), (0, 3, 2), (1, 1, 1)])
def test_every_vg_exactly_once(total, quota, chunk):
    for seed in range(5):
        execs, fetches = D.simulate(total, quota, chunk, seed)
        vgs = sorted(v for _, v in execs)
        assert vgs == list(range(total))
        # one atomic per chunk plus one terminal fetch per CTA (Fig. 8b loop)
        assert fetches == -(-total // chunk) + quota


def test_fig3_assignment_is_dynamic():
    """Fig. 3b: two WGs dequeue A's 12 VGs; the VG->WG mapping varies (lines 456-459)."""
    maps = set()
    for seed in range(20):
        execs, _ = D.simulate(12, 2, 1, seed)
        maps.add(tuple(c for c, _ in sorted(execs, key=lambda e: e[1])))
    assert len(maps) > 1


def test_decode_matches_numpy_unravel():
    gx, gy, gz = 5, 3, 4
    for vg in range(gx * gy * gz):
        z, y, x = np.unravel_index(vg, (gz, gy, gx))
        assert D.decode(vg, gx, gy) == (x, y, z)


def test_shrink_still_covers():
    """Resolve-policy shrink: the live quota drops mid-run; survivors finish."""
    for seed in range(10):
        execs, _ = D.simulate(300, 8, 2, seed, live_quota=lambda step: 8 if step < 40 else 3)
        assert sorted(v for _, v in execs) == list(range(300))
        late = {c for c, v in execs if v >= 200}
        assert late <= set(range(8))
