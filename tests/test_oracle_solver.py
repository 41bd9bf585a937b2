"""Pins for the share-solver oracle (§3).

The oracle is checked against things other than itself: the paper's worked
example (Fig. 3, lines 300-371 / §2.3-2.4), NVIDIA's occupancy calculator
(cuda_occupancy.h) for K = 1, exhaustive enumeration on tiny devices, and the
invariants BASELINE.json's north star names (quotas within per-SM limits,
equal shares for identical kernels).
"""
import itertools
import random

import pytest

from oracle import solver_ref as S


def test_fig3_worked_example():
    """Fig. 3: 4 CUs, kernels A (12 WGs) and B (8 WGs), each CU fits one WG of
    either; accelOS reduces both to 2 WGs (lines 404-408, 441-445), A on
    CU0/CU1 and B on CU2/CU3 (Fig. 3b)."""
    caps = S.Caps(sms=4, thr_per_sm=256, regs_per_sm=65536, smem_per_sm=233472, ctas_per_sm=32)
    a = S.demand_of(256, 32, 0, 12, caps=caps)
    b = S.demand_of(256, 32, 0, 8, caps=caps)
    n = S.solve([a, b], caps)
    assert n == [2, 2]
    # original grids (standard mode) would not fit side by side: A alone takes all 4 CUs
    assert S.solve([a], caps) == [4]
    assert not S.feasible([a, b], [3, 2], caps)


@pytest.mark.parametrize("block,regs,smem", [
    (256, 32, 0), (256, 64, 0), (128, 255, 0), (256, 32, 100000), (96, 40, 0),
    (1024, 32, 0), (128, 72, 16384), (64, 16, 48000), (512, 128, 0), (32, 255, 8000),
    (160, 56, 3000), (256, 40, 40 * 1024), (992, 64, 0), (128, 168, 0),
])
def test_single_kernel_matches_occupancy_calculator(occ, block, regs, smem):
    """K = 1 -> n = min(G, 148 * cudaOccMaxActiveBlocksPerMultiprocessor)."""
    per_sm = occ(block, regs, 0, smem)
    assert per_sm > 0
    for g in (1, 7, 148 * per_sm - 1, 148 * per_sm, 10 ** 6):
        d = S.demand_of(block, regs, smem, g)
        assert S.solve([d]) == [min(g, 148 * per_sm)]


def test_nofit():
    with pytest.raises(S.NoFit):
        S.demand_of(256, 32, 240 * 1024, 10)
    with pytest.raises(S.NoFit):
        S.demand_of(1024, 255, 0, 10)  # 32 warps * 8192 regs > 64K per SM


def test_equal_shares_example():
    """SURVEY §8(c).1 example: 4 identical 256-thread CTAs at 32 regs, no smem:
    296 each = 2 CTAs per SM per kernel."""
    d = S.demand_of(256, 32, 0, 10 ** 6)
    assert S.solve([d] * 4) == [296] * 4


def _random_demand(r, caps, gmax=5000):
    while True:
        block = r.choice([32, 64, 96, 128, 192, 256, 384, 512, 1024])
        regs = r.choice([16, 24, 32, 40, 48, 64, 72, 96, 128, 168, 255])
        smem = r.choice([0, 0, 0, 1024, 4096, 16384, 32768, 49152, 100000])
        try:
            return S.demand_of(block, regs, smem, r.randint(0, gmax), caps=caps)
        except S.NoFit:
            continue


def _check_invariants(ds, n, caps):
    if not S.feasible(ds, [min(1, d.grid_vgs) for d in ds], caps):
        assert n == [min(1, d.grid_vgs) for d in ds]
        return
    assert S.feasible(ds, n, caps)
    for d, q in zip(ds, n):
        assert 0 <= q <= d.grid_vgs
        if d.grid_vgs > 0:
            assert q >= 1
    # identical requests -> identical quotas
    for members in S.classes(ds):
        assert len({n[i] for i in members}) == 1
    # class-maximality: no class can be incremented
    for members in S.classes(ds):
        if all(n[i] + 1 <= ds[i].grid_vgs for i in members):
            m = list(n)
            for i in members:
                m[i] += 1
            assert not S.feasible(ds, m, caps)
    # totals within the device
    T = caps.sms
    assert sum(q * d.thr for d, q in zip(ds, n)) <= T * caps.thr_per_sm
    assert sum(q * d.regs for d, q in zip(ds, n)) <= T * caps.regs_per_sm
    assert sum(q * d.smem for d, q in zip(ds, n)) <= T * caps.smem_per_sm
    assert sum(q for q in n) <= T * caps.ctas_per_sm


def test_random_invariants_b200():
    r = random.Random(7)
    caps = S.Caps()
    for _ in range(30):
        k = r.randint(1, 8)
        ds = [_random_demand(r, caps) for _ in range(k)]
        if r.random() < 0.3:  # duplicate kernels
            ds = ds + [ds[0]] * r.randint(1, 3)
        n = S.solve(ds, caps)
        _check_invariants(ds, n, caps)


def test_identical_kernels_get_equal_quota():
    caps = S.Caps()
    for k in range(1, 9):
        for block, regs, smem in [(128, 40, 0), (256, 64, 8192), (96, 33, 1000)]:
            d = S.demand_of(block, regs, smem, 10 ** 6)
            n = S.solve([d] * k, caps)
            assert len(set(n)) == 1


def test_bruteforce_tiny_devices():
    """Tiny devices: enumerate every n; the greedy result is feasible and
    class-maximal, never exceeds a feasible optimum of the min-share, and
    the closed form is a lower bound whenever it is feasible."""
    r = random.Random(11)
    for trial in range(150):
        caps = S.Caps(sms=r.randint(1, 3), thr_per_sm=r.choice([256, 512, 1024]),
                      regs_per_sm=r.choice([16384, 32768, 65536]),
                      smem_per_sm=r.choice([8192, 16384, 49152]), ctas_per_sm=r.choice([2, 4, 8]))
        k = r.randint(1, 3)
        ds = []
        while len(ds) < k:
            try:
                ds.append(S.demand_of(r.choice([32, 64, 128, 256]), r.choice([16, 32, 64, 128]),
                                      r.choice([0, 1024, 4096, 12000]), r.randint(0, 9), caps=caps))
            except S.NoFit:
                pass
        n = S.solve(ds, caps)
        _check_invariants(ds, n, caps)
        if not S.feasible(ds, n, caps):
            continue
        ranges = [range(0, d.grid_vgs + 1) for d in ds]
        best_min = -1
        for cand in itertools.product(*ranges):
            if any(d.grid_vgs > 0 and c == 0 for d, c in zip(ds, cand)):
                continue
            if S.feasible(ds, list(cand), caps):
                best_min = max(best_min, min(cand) if cand else 0)
        assert best_min >= 0
        assert min(n) <= best_min  # cannot beat the max-min optimum
        cf = S.closed_form(ds, caps)
        if S.feasible(ds, cf, caps):
            assert all(a >= b for a, b in zip(n, cf))


def test_weights_scale_shares():
    """§2.2 (lines 388-393): changing the sharing ratio; weight 2 gets 2x the
    closed-form share of an otherwise identical kernel."""
    a = S.demand_of(256, 32, 0, 10 ** 6, weight=2)
    b = S.demand_of(256, 32, 0, 10 ** 6, weight=1)
    cf = S.closed_form([a, b])
    assert cf == [789, 394]  # floor(148*2048*2/(3*256)), floor(148*2048/(3*256))
    n = S.solve([a, b])
    _check_invariants([a, b], n, S.Caps())


def test_zero_grid_gets_zero():
    a = S.demand_of(256, 32, 0, 0)
    b = S.demand_of(256, 32, 0, 1000)
    assert S.solve([a, b]) == [0, 1000]


def test_step_quota():
    """R-solver-8: a secondary step is solved with its own kernel in place."""
    main = S.demand_of(256, 32, 0, 10 ** 6)
    other = S.demand_of(256, 32, 0, 10 ** 6)
    small = S.demand_of(256, 32, 0, 8)
    assert S.step_quota([main, other], 0, small) == 8
    big_smem = S.demand_of(128, 96, 190 * 1024, 256)
    assert S.step_quota([main, other], 0, big_smem) == 148  # one 191-KB CTA per SM


def test_placement_big_cta_not_starved():
    """R-solver-3 / R-place-1: small CTAs arriving first must not fragment
    every SM.  A GEMM whose CTA needs a whole SM (640 threads x 96 registers)
    beside a small SpMV kernel: by the closed form both get half of the
    registers, i.e. 74 GEMM CTAs (one per SM on half the SMs); the SpMV CTAs
    pack on the other SMs.  (Dealing SpMV's 127 CTAs one per SM first left
    the GEMM 21 SMs.)"""
    g, sp = S.demand_of(640, 96, 189 * 1024, 512), S.demand_of(256, 40, 0, 2304)
    for ds, gi in (([sp, g], 1), ([g, sp], 0)):
        n = S.solve(ds)
        assert n[gi] == 74
        _check_invariants(ds, n, S.Caps())
    # brute-force placement check on a 4-SM toy: a full-SM CTA + three 1/4-SM CTAs
    caps = S.Caps(sms=4, thr_per_sm=1024, regs_per_sm=65536, smem_per_sm=233472, ctas_per_sm=32)
    big, small = S.demand_of(1024, 32, 0, 8, caps=caps), S.demand_of(256, 32, 0, 8, caps=caps)
    assert S.feasible([small, big], [8, 2], caps)        # big on SM0, SM1; small 4 + 4 on SM2, SM3
    assert not S.feasible([small, big], [9, 2], caps)    # 9 quarter-SM CTAs need 3 SMs
