"""Reference of the software work-group scheduling semantics
(TEST INFRASTRUCTURE ONLY -- see oracle/__init__.py).

PAPER.md §2.4 (lines 439-459) and Fig. 8b (lines 748-781), restated: the
original work-groups of a kernel execution are stored as virtual groups (VGs)
in a software queue in accelerator memory (the Virtual NDRange); each of the
reduced number of physical work-groups runs a loop in which a master
work-item dequeues VG(s) atomically, the group synchronises, leaves on
RUN_TERMINATE, and otherwise runs the computation for every VG in
[wg_base, wg_end).  §6.4 (lines 824-834): one dequeue may hand out several
VGs ("adaptive scheduling").  Which physical group runs which VG is not
specified (lines 456-459).

Readings: R-disp-1 the queue of VGs 0..G-1 degenerates to an atomic counter
(dequeue order = increasing linear id, as in Fig. 3b); R-disp-2 multi-dimensional
VG ids decode x-fastest; R-disp-3 a partial last chunk runs [base, G); a CTA
leaves when base >= G or (resolve policy) when its index >= live quota.

`simulate` plays the protocol sequentially under a seeded random interleaving
of CTAs, so tests can check coverage and termination with no GPU.
"""
from __future__ import annotations

import random
from typing import Callable


def decode(vg: int, gx: int, gy: int) -> tuple[int, int, int]:
    """Linear VG id -> (x, y, z), x fastest (R-disp-2)."""
    return vg % gx, (vg // gx) % gy, vg // (gx * gy)


def simulate(total: int, quota: int, chunk: int, seed: int = 0,
             live_quota: Callable[[int], int] | None = None):
    """Run the dequeue loop for `quota` CTAs over `total` VGs.

    live_quota(step) -> current live quota (resolve-policy shrink); default
    constant `quota`.  Returns (executions, fetches) where executions is a list
    of (cta, vg) in execution order and fetches the number of atomic dequeues.
    """
    r = random.Random(seed)
    nxt = 0
    fetches = 0
    alive = list(range(quota))
    pending: dict[int, list[int]] = {c: [] for c in alive}
    execs: list[tuple[int, int]] = []
    step = 0
    while alive:
        c = r.choice(alive)
        step += 1
        if pending[c]:
            execs.append((c, pending[c].pop(0)))
            continue
        lq = quota if live_quota is None else live_quota(step)
        if c >= lq:
            alive.remove(c)
            continue
        base = nxt
        nxt += chunk
        fetches += 1
        if base >= total:
            alive.remove(c)
            continue
        pending[c] = list(range(base, min(base + chunk, total)))
    return execs, fetches
