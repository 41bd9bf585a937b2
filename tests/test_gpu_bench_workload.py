"""GPU parity of the EXACT benchmarked workload, and the placement the solver
assumed, checked on the hardware.

* The C2 mix of bench.py (bfs + cutcp + stencil + tpacf, default sizes, seeds
  3-6; BASELINE config 2), submitted together in
  NATIVE, SHARED-STATIC and SHARED-RESOLVE: every output against the CPU
  oracle (bfs, stencil, tpacf in full; cutcp on sampled lattice points), and
  SHARED bit-identical to NATIVE (output transparency).
* Placement: under SHARED every quota CTA of a request's first launch gets
  work, runs on one SM (%smid), and the per-SM CTA counts the hardware chose
  stay within the per-SM model F the solver assumed (DESIGN.md R-solver-3,
  oracle/solver_ref.placement) and within the SM's resources -- the premise
  of "equal resources per kernel".
"""
import numpy as np
import pytest

from tests.gpu_util import assert_close_fp32

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def c2():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no GPU")
    import bench
    tenants, size, inputs = bench.make_inputs("c2", 0)
    assert tenants == ["bfs", "cutcp", "stencil", "tpacf"] and size == "default"
    return tenants, inputs


@pytest.fixture(scope="module")
def c2_refs(c2, oracle_lib):
    _, d = c2
    r = np.random.Generator(np.random.PCG64(11))
    dc = d["cutcp"]
    ijk = np.stack([r.integers(0, dc["nx"], 4000), r.integers(0, dc["ny"], 4000), r.integers(0, dc["nz"], 4000)], 1)
    return {"bfs": oracle_lib.bfs(d["bfs"]), "stencil": oracle_lib.stencil(d["stencil"]),
            "tpacf": oracle_lib.tpacf(d["tpacf"]), "cutcp": (ijk, oracle_lib.cutcp_points(dc, ijk))}


def _check(jobs, refs):
    lv, depth = refs["bfs"]
    assert depth + 1 <= jobs[0].levels                      # the request covers every level
    assert np.array_equal(jobs[0].result()["level"], lv)
    ijk, ref = refs["cutcp"]
    v = jobs[1].result()["v"][ijk[:, 2], ijk[:, 1], ijk[:, 0]]
    assert np.array_equal(v == 0, ref == 0)
    assert_close_fp32(v, ref, what="cutcp (C2)")
    assert_close_fp32(jobs[2].result()["a"], refs["stencil"], what="stencil (C2)")
    t = jobs[3].result()
    dd, rr, dr = refs["tpacf"]
    assert np.array_equal(t["dd"], dd) and np.array_equal(t["rr"], rr) and np.array_equal(t["dr"], dr)


def test_c2_bench_workload_every_mode(c2, c2_refs):
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import make_job
    from paper_conf_cgo_margiolaso16_b200.runtime import Accel
    tenants, d = c2
    outs = {}
    with Accel(device=0, mode=abi.MODE_SHARED, verify=True) as acc:
        for name, mode, pol in [("native", abi.MODE_NATIVE, abi.POLICY_STATIC),
                                ("static", abi.MODE_SHARED, abi.POLICY_STATIC),
                                ("resolve", abi.MODE_SHARED, abi.POLICY_RESOLVE)]:
            acc.set_mode(mode, pol)
            jobs = [make_job(t, d[t]) for t in tenants]
            st = acc.run(jobs)
            assert all(s.coverage_ok == 1 for s in st), name
            _check(jobs, c2_refs)
            outs[name] = [j.result() for j in jobs]
    for name in ("static", "resolve"):
        for a, b in zip(outs["native"], outs[name]):
            for k in a:
                assert np.array_equal(a[k], b[k]), (name, k)


@pytest.mark.parametrize("policy", ["static", "resolve"])
def test_c2_placement_matches_solver_model(c2, policy):
    import torch

    from oracle import solver_ref as S
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import make_job
    from paper_conf_cgo_margiolaso16_b200.runtime import Accel
    tenants, d = c2
    n_sm = torch.cuda.get_device_properties(0).multi_processor_count
    pol = abi.POLICY_STATIC if policy == "static" else abi.POLICY_RESOLVE
    with Accel(device=0, mode=abi.MODE_SHARED, policy=pol) as acc:
        jobs = [make_job(t, d[t]) for t in tenants]
        ids = acc.submit(jobs, trace=True)
        acc.sync()
        st = [acc.stats(i) for i in ids]
        tr = [acc.vg_trace(i) for i in ids]
        infos = [acc.kernel_info(j.steps[j.main_step].kernel) for j in jobs]
        acc.release()
    quotas = [s.quota_initial for s in st]
    # the solver's model of the same group (demands as the library computed them)
    ds = [S.Demand(thr=i.thr, regs=i.regs, smem=i.smem, cta=i.cta, grid_vgs=int(np.prod(j.steps[j.main_step].grid)))
          for i, j in zip(infos, jobs)]
    assert S.solve(ds, S.Caps(sms=n_sm)) == quotas        # the library solved what the oracle solves
    model = S.placement(ds, quotas, S.Caps(sms=n_sm))
    assert model is not None, "the solver's quotas must be feasible under its own model"
    fmax = [max(row[i] for row in model) for i in range(len(ds))]
    hw = np.zeros((n_sm, len(ds)), dtype=np.int64)
    for i, t in enumerate(tenants):
        if t == "bfs":
            continue   # its first launch has one VG: most of its CTAs get no work to trace
        g0 = int(np.prod(jobs[i].steps[0].grid))
        rec = tr[i][:g0]
        rec = rec[(rec["t_start_ns"] > 0) & (rec["cta"] < 0x80000000)]   # main-grid CTAs
        ctas = np.unique(rec["cta"])
        assert len(ctas) == quotas[i], (t, len(ctas), quotas[i])        # every quota CTA got work
        sm_of = {}
        for c, sm in zip(rec["cta"], rec["sm"]):
            assert sm_of.setdefault(int(c), int(sm)) == int(sm), "a CTA never migrates"
        for c, sm in sm_of.items():
            hw[sm, i] += 1
        # every CTA of the launch started before any CTA of it retired: the
        # whole quota was resident at once
        first = np.array([rec["t_start_ns"][rec["cta"] == c].min() for c in ctas])
        last = np.array([rec["t_end_ns"][rec["cta"] == c].max() for c in ctas])
        assert first.max() <= last.min(), (t, int(first.max() - last.min()))
        assert hw[:, i].max() <= fmax[i], (t, int(hw[:, i].max()), fmax[i])
    # co-resident CTAs of the traced requests fit every SM's resources
    caps = S.Caps(sms=n_sm)
    for sm in range(n_sm):
        assert sum(hw[sm, i] * ds[i].thr for i in range(len(ds))) <= caps.thr_per_sm
        assert sum(hw[sm, i] * ds[i].smem for i in range(len(ds))) <= caps.smem_per_sm
        assert sum(hw[sm, i] * ds[i].regs for i in range(len(ds))) <= caps.regs_per_sm
