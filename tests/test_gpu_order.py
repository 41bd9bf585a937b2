"""GPU: the library's cost-model dequeue order (DESIGN.md R-disp-7,
dispatch.cuh accel_lpt_order) -- VG ids by decreasing T::vg_cost, ties by
increasing id -- against an independent numpy model of the same costs (the
atoms a cutcp VG streams, the Q tiles a tpacf VG walks), and the order is a
permutation (so coverage cannot change).  The software queue may hand VGs
out in any order; correctness never depends on it."""
import numpy as np
import pytest

import synth

pytestmark = pytest.mark.gpu


def _lpt(cost):
    return np.argsort(-np.asarray(cost, dtype=np.float64), kind="stable")


def cutcp_cost(d, grid):
    """Atoms streamed per VG: the cell rows and trimmed x-ranges the body walks
    (tenants/cutcp.cuh), in float32 like the device."""
    f = np.float32
    gx, gy, gz = grid
    h, cs, nc = f(d["h"]), f(d["cell"]), int(d["ncell_1d"])
    cm = f(f(d["cutoff"]) + f(0.05))
    cst = np.asarray(d["cell_start"], dtype=np.int64)
    cost = np.zeros(gx * gy * gz)
    cl = lambda v: min(max(v, 0), nc - 1)  # noqa: E731
    gap = lambda lo, hi, clo, chi: max(f(0), max(f(clo - hi), f(lo - chi)))  # noqa: E731
    for v in range(gx * gy * gz):
        x, y, z = v % gx, (v // gx) % gy, v // (gx * gy)
        b0 = [f(h * f(8 * c)) for c in (x, y, z)]
        b1 = [f(h * f(8 * c + 7)) for c in (x, y, z)]
        cy0, cy1 = cl(int(np.floor(f(f(b0[1] - cm) / cs)))), cl(int(np.floor(f(f(b1[1] + cm) / cs))))
        cz0, cz1 = cl(int(np.floor(f(f(b0[2] - cm) / cs)))), cl(int(np.floor(f(f(b1[2] + cm) / cs))))
        tot = 0
        for cz in range(cz0, cz1 + 1):
            gzv = gap(b0[2], b1[2], f(cz * cs), f((cz + 1) * cs))
            for cy in range(cy0, cy1 + 1):
                gyv = gap(b0[1], b1[1], f(cy * cs), f((cy + 1) * cs))
                d2 = f(f(gyv * gyv) + f(gzv * gzv))
                if d2 >= f(cm * cm):
                    continue
                rx = np.sqrt(f(f(cm * cm) - d2), dtype=np.float32)
                cx0 = cl(int(np.floor(f(f(b0[0] - rx) / cs))))
                cx1 = cl(int(np.floor(f(f(b1[0] + rx) / cs))))
                row = (cz * nc + cy) * nc
                tot += cst[row + cx1 + 1] - cst[row + cx0]
        cost[v] = tot
    return cost


def tpacf_cost(S, n, grid):
    """Q tiles per VG (x, y, part z): part z of the tiles from the diagonal
    one (DD/RR, y <= S) or from tile 0 (DR), the diagonal tile half-counted."""
    gx, gy, gz = grid
    ntiles = -(-n // 256)
    cost = np.zeros(gx * gy * gz)
    for v in range(gx * gy * gz):
        x, y, z = v % gx, (v // gx) % gy, v // (gx * gy)
        first = x if y <= S else 0
        ln = ntiles - first
        t0, t1 = first + ln * z // gz, first + ln * (z + 1) // gz
        cost[v] = (t1 - t0) - (0.5 if (y <= S and t0 == x and t1 > t0) else 0.0)
    return cost


@pytest.mark.parametrize("tenant,size", [("cutcp", "tiny"), ("cutcp", "small"), ("tpacf", "tiny"),
                                         ("tpacf", "default")])
def test_library_order_is_lpt_of_the_cost_model(tenant, size):
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no GPU")
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import make_job
    from paper_conf_cgo_margiolaso16_b200.runtime import Accel
    d = synth.preset(tenant, size, seed=2)
    job = make_job(tenant, d)
    st = job.steps[0]
    g = int(np.prod(st.grid))
    out = torch.full((g,), -1, dtype=torch.int32, device="cuda")
    with Accel(device=0, mode=abi.MODE_SHARED) as acc:
        torch.cuda.synchronize()
        abi.accel_dequeue_order(acc.ctx, acc.kids[st.kernel], st.grid, st.args, out.data_ptr())
        got = out.cpu().numpy().astype(np.int64)
    assert np.array_equal(np.sort(got), np.arange(g))             # a permutation
    cost = cutcp_cost(d, st.grid) if tenant == "cutcp" else tpacf_cost(d["nsets"], d["npts"], st.grid)
    # non-increasing cost along the order, ties by increasing id
    c = cost[got]
    assert (np.diff(c) <= 0).all()
    same = np.diff(c) == 0
    assert (np.diff(got)[same] > 0).all()
    assert np.array_equal(got, _lpt(cost))


def test_linear_order_flag_keeps_results():
    """ACCEL_REQ_LINEAR_ORDER (no cost model) and the default order give the
    same bit-exact output (any dequeue order is correct)."""
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no GPU")
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import make_job
    from paper_conf_cgo_margiolaso16_b200.runtime import Accel
    d = synth.preset("cutcp", "small", seed=3)
    outs = []
    with Accel(device=0, mode=abi.MODE_SHARED, verify=True) as acc:
        for lin in (False, True):
            job = make_job("cutcp", d)
            ids = acc.submit([job], linear_order=lin)
            acc.sync()
            assert acc.stats(ids[0]).coverage_ok == 1
            acc.release()
            outs.append(job.result()["v"])
    assert np.array_equal(outs[0], outs[1])
