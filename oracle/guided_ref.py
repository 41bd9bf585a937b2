"""Reference profile-guided sharing ratios (TEST INFRASTRUCTURE ONLY -- see
oracle/__init__.py).

DESIGN.md R-solver-11, an extension of PAPER.md lines 388-393 ("changing the
sharing ratio"), restated step by step:
  1. s_i(f_j) = max(1, T_i(f_j) / T_i(1)) at the profiled fractions, then made
     non-increasing in f (s at a fraction = max of s at every larger
     measured fraction... i.e. a running max from f = 1 downwards), s_i(1) = 1;
  2. between profiled fractions s_i is a power law (linear in log f, log s);
     below the smallest one it scales as 1/f; at f >= 1 it is 1;
  3. f_i(S) = min { f in (0, 1] : s_i(f) <= S };
  4. S = min { S >= 1 : sum_i f_i(S) <= 1 }  (found by bisection);
  5. w_i = max(1, round(scale * f_i(S) / max_j f_j(S))).
Plain Python, no shared code with csrc/host/guided.cpp.
"""
from __future__ import annotations

import math


def slowdown_curve(fracs, ms):
    """(ascending fractions, non-increasing slowdowns) of one profile."""
    pts = sorted(zip(fracs, ms))                  # ascending f
    t1 = dict(zip(fracs, ms))[1.0]
    f = [p[0] for p in pts]
    s = [max(1.0, p[1] / t1) for p in pts]
    for j in range(len(s) - 2, -1, -1):          # running max from f = 1 down
        s[j] = max(s[j], s[j + 1])
    s[-1] = 1.0
    return f, s


def slowdown_at(f, s, x):
    if x >= 1.0:
        return 1.0
    if x <= f[0]:
        return s[0] * f[0] / x
    for j in range(1, len(f)):
        if x <= f[j]:
            e = math.log(s[j] / s[j - 1]) / math.log(f[j] / f[j - 1])
            return s[j - 1] * (x / f[j - 1]) ** e
    return 1.0


def fraction_for(f, s, S):
    """Smallest x in (0, 1] with slowdown_at(x) <= S, by definition: the
    curve is continuous and non-increasing, so it is where it crosses S."""
    if S >= s[0]:
        return min(1.0, s[0] * f[0] / S)
    for j in range(1, len(f)):
        if s[j] <= S:   # s[j-1] > S >= s[j]
            e = math.log(s[j] / s[j - 1]) / math.log(f[j] / f[j - 1])
            return min(f[j], f[j - 1] * (S / s[j - 1]) ** (1.0 / e))
    return 1.0


def guided_weights(fracs, ms, scale=16):
    curves = [slowdown_curve(fracs, row) for row in ms]
    total = lambda S: sum(fraction_for(f, s, S) for f, s in curves)  # noqa: E731
    lo = hi = 1.0
    if total(1.0) > 1.0:
        hi = 2.0
        while total(hi) > 1.0:
            hi *= 2.0
        for _ in range(200):
            mid = 0.5 * (lo + hi)
            if total(mid) > 1.0:
                lo = mid
            else:
                hi = mid
    S = hi
    fr = [fraction_for(f, s, S) for f, s in curves]
    fmax = max(fr)
    w = [max(1, int(round(scale * x / fmax))) for x in fr]
    pred = [slowdown_at(f, s, x) for (f, s), x in zip(curves, fr)]
    return w, pred, S, fr
