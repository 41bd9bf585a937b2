"""The product solver (C++ accel_solve in libaccel.so) equals the oracle
(oracle/solver_ref.py) exactly; demand vectors and metrics likewise."""
import math
import random

import pytest

from oracle import metrics_ref as M
from oracle import solver_ref as S
from paper_conf_cgo_margiolaso16_b200 import abi


def _caps(c: S.Caps) -> abi.accel_caps:
    return abi.accel_caps(c.sms, c.thr_per_sm, c.regs_per_sm, c.smem_per_sm, c.ctas_per_sm)


def _to_c(d: S.Demand) -> abi.accel_demand:
    return abi.accel_demand(d.thr, d.regs, d.smem, d.cta, d.grid_vgs, d.weight)


def test_demand_vectors_equal():
    r = random.Random(1)
    for _ in range(3000):
        block = r.randint(1, 1024)
        regs = r.randint(1, 255)
        smem = r.choice([0, r.randint(0, 240 * 1024)])
        g = r.randint(0, 10 ** 6)
        try:
            ref = S.demand_of(block, regs, smem, g)
        except S.NoFit:
            with pytest.raises(abi.AccelError):
                abi.accel_demand_of(block, regs, smem, g)
            continue
        d = abi.accel_demand_of(block, regs, smem, g)
        assert (d.thr, d.regs, d.smem, d.cta, d.grid_vgs, d.weight) == ref.key()


def _random_instance(r, caps, kmax, gmax):
    ds = []
    k = r.randint(1, kmax)
    while len(ds) < k:
        try:
            ds.append(S.demand_of(r.choice([32, 64, 96, 128, 192, 256, 512, 1024]),
                                  r.choice([16, 24, 32, 40, 48, 64, 80, 96, 128, 168, 255]),
                                  r.choice([0, 0, 1024, 4096, 10240, 16384, 49152, 100000]),
                                  r.randint(0, gmax), r.choice([1, 1, 1, 2, 3]), caps=caps))
        except S.NoFit:
            pass
    if r.random() < 0.3:
        ds += [ds[0]] * r.randint(1, 3)
    return ds


def test_parity_tiny_devices():
    r = random.Random(2)
    n = 0
    for _ in range(6000):
        caps = S.Caps(sms=r.randint(1, 9), thr_per_sm=r.choice([512, 1024, 2048]),
                      regs_per_sm=r.choice([32768, 65536]), smem_per_sm=r.choice([65536, 233472]),
                      ctas_per_sm=r.choice([4, 8, 16, 32]))
        try:
            ds = _random_instance(r, caps, 4, 40)
        except S.NoFit:
            continue
        ref = S.solve(ds, caps)
        got = abi.accel_solve([_to_c(d) for d in ds], _caps(caps))
        assert got == ref, (caps, ds)
        n += 1
    assert n > 5000


def test_parity_b200():
    r = random.Random(3)
    caps = S.Caps()
    for _ in range(40):   # the oracle's placement simulation is slow in Python
        ds = _random_instance(r, caps, 8, 20000)
        assert abi.accel_solve([_to_c(d) for d in ds]) == S.solve(ds, caps)


def test_fig3_toy_in_product():
    caps = S.Caps(sms=4, thr_per_sm=256)
    a = S.demand_of(256, 32, 0, 12, caps=caps)
    b = S.demand_of(256, 32, 0, 8, caps=caps)
    assert abi.accel_solve([_to_c(a), _to_c(b)], _caps(caps)) == [2, 2]


def test_metrics_equal():
    r = random.Random(4)
    for _ in range(500):
        k = r.randint(1, 8)
        ta = [r.uniform(0.1, 10) for _ in range(k)]
        ts = [a * r.uniform(1, 20) for a in ta]
        m = abi.accel_metrics(ta, ts)
        assert m.unfairness == pytest.approx(M.unfairness(ts, ta), rel=1e-12)
        assert m.stp == pytest.approx(M.stp(ts, ta), rel=1e-12)
        assert m.antt == pytest.approx(M.antt(ts, ta), rel=1e-12)
        st = [r.uniform(0, 5) for _ in range(k)]
        en = [s + r.uniform(0, 5) for s in st]
        assert abi.accel_overlap(st, en) == pytest.approx(M.overlap(list(zip(st, en))), abs=1e-12)


def test_placement_order_parity():
    """R-place-1: the library's enqueue / placement order equals the oracle's
    (largest per-CTA footprint first, ties in arrival order)."""
    r = random.Random(21)
    caps = S.Caps()
    for _ in range(300):
        ds = _random_instance(r, caps, 8, 5000)
        assert abi.accel_placement_order([_to_c(d) for d in ds]) == S.placement_order(ds, caps)
    # a one-CTA-per-SM GEMM (registers) goes before a small SpMV CTA whatever the arrival order
    g, sp = S.demand_of(640, 96, 189 * 1024, 512), S.demand_of(256, 40, 0, 2304)
    assert S.placement_order([sp, g]) == [1, 0]
    assert abi.accel_placement_order([_to_c(sp), _to_c(g)]) == [1, 0]


def test_weighted_metrics_equal():
    """libaccel accel_metrics_weighted == oracle/metrics_ref (R-metric-5)."""
    r = random.Random(9)
    for _ in range(300):
        k = r.randint(1, 8)
        ta = [r.uniform(0.1, 5) for _ in range(k)]
        ts = [a * r.uniform(1, 6) for a in ta]
        w = [r.choice([1, 2, 3, 16, 0.5]) for _ in range(k)]
        wu, ws = abi.accel_metrics_weighted(ta, ts, w)
        assert wu == pytest.approx(M.weighted_unfairness(ts, ta, w), rel=1e-12)
        assert ws == pytest.approx(M.weighted_slowdown(ts, ta, w), rel=1e-12)


def test_solve_memo_consistent():
    """accel_solve memoises by (caps, demands) (solver.cpp): a repeated
    instance -- with other instances solved in between -- returns its first
    answer, which equals the oracle."""
    r = random.Random(77)
    caps = S.Caps(sms=6)
    inst = []
    while len(inst) < 8:
        try:
            inst.append(_random_instance(r, caps, 4, 40))
        except S.NoFit:
            continue
    first = [abi.accel_solve([_to_c(d) for d in ds], _caps(caps)) for ds in inst]
    again = [abi.accel_solve([_to_c(d) for d in ds], _caps(caps)) for ds in reversed(inst)][::-1]
    assert first == again
    for ds, q in zip(inst, first):
        assert q == S.solve(ds, caps)
