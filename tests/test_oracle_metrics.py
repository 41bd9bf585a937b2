"""Pins for the metrics oracle (§7.4, §8 results).

The paper prints unfairness values and the fairness improvements derived from
them; the oracle's formulas must reproduce the paper's own arithmetic.
"""
import math

import pytest

from oracle import metrics_ref as M


@pytest.mark.parametrize("u_std,u_acc,printed", [
    (8.43, 1.24, 6.8),     # NV, 2 requests (lines 929-934)
    (19.65, 1.89, 10.4),   # NV, 4 requests
    (43.42, 3.54, 12.27),  # NV, 8 requests
    (12.97, 1.58, 8.21),   # AMD, 2 requests (lines 944-947)
    (31.25, 3.27, 9.56),   # AMD, 4 requests
])
def test_fairness_improvement_matches_paper(u_std, u_acc, printed):
    assert M.fairness_improvement(u_std, u_acc) == pytest.approx(printed, abs=0.01)


def test_amd_8_request_ratio_is_not_13_66():
    """Lines 949-950 print 13.66x for 28.57 -> 2.79, but the ratio of those
    means is 10.24x (DESIGN.md R-metric-3: per-mix FI means and ratios of
    mean U differ); the oracle reports the ratio."""
    assert M.fairness_improvement(28.57, 2.79) == pytest.approx(10.24, abs=0.01)


@pytest.mark.parametrize("xs,printed,tol", [
    ((6.8, 10.4, 12.27), 9.55, 0.015),   # accelOS NV average (line 934)
    ((1.53, 1.03, 0.93), 1.13, 0.01),    # EK NV average (lines 936-937)
    ((1.63, 0.77, 0.85), 1.02, 0.005),   # EK AMD average (lines 950-952)
    ((1.13, 1.19, 1.23), 1.18, 0.005),   # accelOS NV throughput (lines 1037-1043)
    ((1.08, 1.02, 0.91), 1.00, 0.005),   # EK NV throughput
    ((1.17, 1.19, 1.31), 1.22, 0.005),   # accelOS AMD throughput (lines 1044-1048)
    ((1.07, 0.95, 0.9), 0.97, 0.005),    # EK AMD throughput
])
def test_averages_are_geometric_means(xs, printed, tol):
    assert M.geomean(xs) == pytest.approx(printed, abs=tol)


def test_arithmetic_mean_would_not_match():
    assert abs(sum((6.8, 10.4, 12.27)) / 3 - 9.55) > 0.2


def test_isolation_is_fair():
    ta = [1.0, 2.0, 5.0]
    assert M.unfairness(ta, ta) == 1.0
    assert M.stp(ta, ta) == 3.0
    assert M.antt(ta, ta) == 1.0


def test_fcfs_example():
    """Fig. 3a / §2.3: A (12 WGs) runs first on all 4 CUs, B (8 WGs) waits.
    With unit WG time: A isolated 3, B isolated 2; shared FCFS: A 3, B 5."""
    ta = [3.0, 2.0]
    ts_fcfs = [3.0, 5.0]
    assert M.unfairness(ts_fcfs, ta) == pytest.approx(2.5)
    # accelOS Fig. 3b: 2 CUs each -> A takes 6, B takes 4: equal slowdown 2
    ts_acc = [6.0, 4.0]
    assert M.unfairness(ts_acc, ta) == pytest.approx(1.0)
    assert M.fairness_improvement(M.unfairness(ts_fcfs, ta), M.unfairness(ts_acc, ta)) == 2.5
    assert M.throughput_speedup(5.0, 6.0) == pytest.approx(5 / 6)


def test_stp_antt_am_hm():
    """STP >= K / ANTT (AM-HM), equality iff all slowdowns are equal."""
    ta = [1.0, 3.0, 2.0, 7.0]
    ts = [2.0, 3.5, 9.0, 7.5]
    k = len(ta)
    assert M.stp(ts, ta) >= k / M.antt(ts, ta) - 1e-12
    ts_eq = [2 * a for a in ta]
    assert M.stp(ts_eq, ta) == pytest.approx(k / M.antt(ts_eq, ta))


def test_overlap():
    assert M.overlap([(0, 10), (0, 10)]) == 1.0
    assert M.overlap([(0, 10), (10, 20)]) == 0.0
    assert M.overlap([(0, 10), (5, 15)]) == pytest.approx(5 / 15)
    assert M.overlap([(0, 10), (2, 4), (3, 12)]) == pytest.approx(1 / 12)
    # gap in the union
    assert M.overlap([(0, 2), (5, 6)]) == 0.0
    assert M.overlap([(0, 4), (1, 3)]) == pytest.approx(0.5)


def test_geomean_closed_form():
    assert M.geomean([2.0, 8.0]) == pytest.approx(4.0)
    assert M.geomean([3.0]) == pytest.approx(3.0)
    assert M.geomean([10.0, 0.1]) == pytest.approx(1.0)
    assert math.isclose(M.geomean([1.5] * 7), 1.5)


# ---- weighted sharing (DESIGN.md R-metric-5) --------

def test_weighted_unfairness_equal_weights_is_unfairness():
    ta, ts = [1.0, 2.0, 0.5], [3.0, 2.5, 2.0]
    for w in ([1, 1, 1], [7, 7, 7]):
        assert M.weighted_unfairness(ts, ta, w) == pytest.approx(M.unfairness(ts, ta))


def test_weighted_unfairness_honoured_ratio_is_one():
    """Two equal jobs, ratio 2:1.  Weighted processor sharing on a fluid
    device: A (weight 2) runs at 2/3 of the device until it finishes at 1.5,
    B at 1/3 until then (0.5 done) and alone after (done at 2.0): IS = 1.5 and
    2.0 -- the LATER job is still favoured less than 2x because B runs alone
    at the end.  WU is the measure: with the ratio honoured throughout (both
    finish in proportion, IS = 1.5 and 3), WS = 1.5*2/1.5 = 2 = 3*1/1.5."""
    assert M.weighted_unfairness([1.5, 3.0], [1.0, 1.0], [2, 1]) == pytest.approx(1.0)
    assert M.weighted_slowdown([1.5, 3.0], [1.0, 1.0], [2, 1]) == pytest.approx([2.0, 2.0])
    # the fluid schedule above is not weighted-fair: WS = [2, 4/3]
    assert M.weighted_unfairness([1.5, 2.0], [1.0, 1.0], [2, 1]) == pytest.approx(1.5)


def test_weighted_unfairness_scale_invariant():
    ta, ts, w = [1.0, 2.0, 4.0], [2.0, 5.0, 6.0], [1.0, 3.0, 2.0]
    a = M.weighted_unfairness(ts, ta, w)
    assert M.weighted_unfairness(ts, ta, [10 * x for x in w]) == pytest.approx(a)
    assert M.weighted_unfairness([3 * x for x in ts], ta, w) == pytest.approx(a)
