"""Reference sharing metrics (TEST INFRASTRUCTURE ONLY -- see oracle/__init__.py).

PAPER.md §7.4 "Metrics" (lines 877-913), restated:
  IS_i = T(s)_i / T(a)_i                       individual slowdown (881-885)
  U    = max_i IS_i / min_i IS_i               system unfairness [9] (886-888)
  FI   = U_baseline / U_X                      fairness improvement (889-894)
  O    = T(c) / T(t)                           kernel execution overlap (895-900)
  speedup = T_baseline / T_X                   makespan ratio (901-908)
  STP, ANTT: named (911-913) but not printed; DESIGN.md R-metric-2 reads them
  as Eyerman & Eeckhout's STP = sum_i T(a)_i/T(s)_i, ANTT = mean_i T(s)_i/T(a)_i.
Weighted sharing (DESIGN.md R-metric-5, "changing the
sharing ratio"): request i is entitled to the share w_i / sum(w), so under
weighted sharing its slowdown should scale as 1 / w_i; the weighted slowdown
WS_i = IS_i * w_i / mean(w) is equal across requests when the sharing honours
the ratios, and WU = max WS / min WS is the weighted unfairness (U when all
weights are equal).
Averages across mixes / request sizes are geometric means (R-metric-3: the
printed 9.55x average of 6.8x, 10.4x, 12.27x is their geometric mean).
"""
from __future__ import annotations

import math
from typing import Sequence


def individual_slowdown(ts: Sequence[float], ta: Sequence[float]) -> list[float]:
    return [s / a for s, a in zip(ts, ta)]


def unfairness(ts: Sequence[float], ta: Sequence[float]) -> float:
    IS = individual_slowdown(ts, ta)
    return max(IS) / min(IS)


def fairness_improvement(u_baseline: float, u_x: float) -> float:
    return u_baseline / u_x


def stp(ts: Sequence[float], ta: Sequence[float]) -> float:
    return sum(a / s for s, a in zip(ts, ta))


def antt(ts: Sequence[float], ta: Sequence[float]) -> float:
    IS = individual_slowdown(ts, ta)
    return sum(IS) / len(IS)


def weighted_slowdown(ts: Sequence[float], ta: Sequence[float], w: Sequence[float]) -> list[float]:
    wbar = sum(w) / len(w)
    return [s / a * wi / wbar for s, a, wi in zip(ts, ta, w)]


def weighted_unfairness(ts: Sequence[float], ta: Sequence[float], w: Sequence[float]) -> float:
    ws = weighted_slowdown(ts, ta, w)
    return max(ws) / min(ws)


def throughput_speedup(makespan_baseline: float, makespan_x: float) -> float:
    return makespan_baseline / makespan_x


def overlap(intervals: Sequence[tuple[float, float]]) -> float:
    """O = T(c)/T(t): T(t) = measure of the union of the [start, end) execution
    intervals (at least one kernel executing), T(c) = time ALL kernels execute
    together (R-metric-4: strict reading, every request has started and none
    has finished)."""
    iv = sorted((float(a), float(b)) for a, b in intervals if b > a)
    if not iv:
        return 0.0
    total = 0.0
    cur_a, cur_b = iv[0]
    for a, b in iv[1:]:
        if a > cur_b:
            total += cur_b - cur_a
            cur_a, cur_b = a, b
        else:
            cur_b = max(cur_b, b)
    total += cur_b - cur_a
    if len(iv) != len(intervals):
        return 0.0
    common = min(b for _, b in iv) - max(a for a, _ in iv)
    return max(0.0, common) / total if total > 0 else 0.0


def geomean(xs: Sequence[float]) -> float:
    return math.exp(sum(math.log(x) for x in xs) / len(xs))
