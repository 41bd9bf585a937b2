"""Pins for liboracle's tenant definitions: closed forms, invariants, library
routines (numpy / scipy / networkx) and brute force on tiny inputs -- never the
oracle's own formula retyped."""
import numpy as np
import pytest

import synth
from synth import gen

pytestmark = pytest.mark.usefixtures("oracle_lib")


def T():
    from oracle import tenants
    return tenants


# ---------------------------------------------------------------- mop
@pytest.mark.parametrize("nconst", [0, 1, 11, 36, 37, 1000])
def test_mop_group_dependence(nconst):
    d = synth.preset("mop", "tiny", nconst=nconst)
    out = T().mop(d)
    g = np.arange(d["n"]) // d["block"]
    ref = np.where(g < nconst, d["ina"] + d["inb"], d["ina"] - d["inb"])
    assert np.array_equal(out, ref)


# ---------------------------------------------------------------- stencil
def _quad_field(nx, ny, nz):
    z, y, x = np.meshgrid(np.arange(nz), np.arange(ny), np.arange(nx), indexing="ij")
    return (x * x + 2 * y * y + 3 * z * z).astype(np.float32)


def test_stencil_quadratic_closed_form():
    """f = x^2 + 2y^2 + 3z^2: the 6-neighbour sum is 6f + 2(1+2+3), so one
    sweep with c0 = 1/6, c1 = 1/36 gives exactly 12/36 = 1/3 inside."""
    nx, ny, nz = 9, 7, 6
    d = {"a0": _quad_field(nx, ny, nz), "nx": nx, "ny": ny, "nz": nz, "sweeps": 1,
         "c0": 1.0 / 6.0, "c1": 1.0 / 36.0}
    out = T().stencil(d)
    assert np.allclose(out[1:-1, 1:-1, 1:-1], 1.0 / 3.0, rtol=0, atol=1e-12)
    f = d["a0"].astype(np.float64)
    for sl in [np.s_[0], np.s_[-1], np.s_[:, 0], np.s_[:, -1], np.s_[:, :, 0], np.s_[:, :, -1]]:
        assert np.array_equal(out[sl], f[sl])


def test_stencil_matches_scipy_correlate():
    """Several sweeps vs scipy.ndimage.correlate with the 7-point kernel,
    boundary faces held at the input values."""
    from scipy import ndimage
    d = synth.preset("stencil", "tiny", sweeps=4)
    k = np.zeros((3, 3, 3))
    k[0, 1, 1] = k[2, 1, 1] = k[1, 0, 1] = k[1, 2, 1] = k[1, 1, 0] = k[1, 1, 2] = d["c1"]
    k[1, 1, 1] = -d["c0"]
    a = d["a0"].astype(np.float64)
    for _ in range(d["sweeps"]):
        b = ndimage.correlate(a, k, mode="nearest")
        b[0], b[-1] = a[0], a[-1]
        b[:, 0], b[:, -1] = a[:, 0], a[:, -1]
        b[:, :, 0], b[:, :, -1] = a[:, :, 0], a[:, :, -1]
        a = b
    assert np.allclose(T().stencil(d), a, rtol=1e-12, atol=1e-14)


# ---------------------------------------------------------------- histo
@pytest.mark.parametrize("size,over", [("tiny", {}), ("tiny", dict(bins=4096, sample_bytes=4)),
                                       ("small", {})])
def test_histo_bincount(size, over):
    d = synth.preset("histo", size, **over)
    counts, sat = T().histo(d)
    ref = np.bincount(d["samples"].astype(np.int64), minlength=d["bins"])
    assert np.array_equal(counts, ref)
    assert counts.sum() == d["n"]
    assert np.array_equal(sat, np.minimum(ref, 255))


# ---------------------------------------------------------------- bfs
def test_bfs_networkx():
    import networkx as nx
    d = synth.preset("bfs", "tiny")
    level, depth = T().bfs(d)
    g = nx.DiGraph()
    g.add_nodes_from(range(d["nv"]))
    rp, col = d["row_ptr"], d["col"]
    for u in range(d["nv"]):
        g.add_edges_from((u, int(w)) for w in col[rp[u]:rp[u + 1]])
    ref = np.full(d["nv"], -1, dtype=np.int32)
    for v, l in nx.single_source_shortest_path_length(g, d["src"]).items():
        ref[v] = l
    assert np.array_equal(level, ref)
    assert depth == ref.max()


def bfs_certificate(d, level):
    """level[src] = 0; every edge u->v from a reached u has 0 <= level[v] <=
    level[u] + 1; every v with level[v] > 0 has an in-edge from level[v]-1;
    unreached vertices have no in-edge from a reached vertex."""
    rp = d["row_ptr"].astype(np.int64)
    col = d["col"].astype(np.int64)
    src = np.repeat(np.arange(d["nv"]), np.diff(rp))
    assert level[d["src"]] == 0
    lu, lv = level[src], level[col]
    reached = lu >= 0
    assert np.all(lv[reached] >= 0)
    assert np.all(lv[reached] <= lu[reached] + 1)
    parent_ok = np.zeros(d["nv"], dtype=bool)
    tight = reached & (lv == lu + 1)
    parent_ok[col[tight]] = True
    need = level > 0
    assert np.all(parent_ok[need])
    return True


def test_bfs_certificate_small():
    d = synth.preset("bfs", "small", seed=3)
    level, _ = T().bfs(d)
    assert bfs_certificate(d, level)


def test_bfs_scipy():
    from scipy.sparse import csr_matrix
    from scipy.sparse.csgraph import shortest_path
    d = synth.preset("bfs", "small", seed=5, src=17)
    level, _ = T().bfs(d)
    m = csr_matrix((np.ones(d["ne"]), d["col"], d["row_ptr"].astype(np.int64)),
                   shape=(d["nv"], d["nv"]))
    sp = shortest_path(m, unweighted=True, indices=d["src"])
    ref = np.where(np.isinf(sp), -1, sp).astype(np.int32)
    assert np.array_equal(level, ref)


# ---------------------------------------------------------------- cutcp
def _lattice(nx, ny, nz):
    k, j, i = np.meshgrid(np.arange(nz), np.arange(ny), np.arange(nx), indexing="ij")
    return np.stack([i.ravel(), j.ravel(), k.ravel()], axis=1).astype(np.int32)


def test_cutcp_single_atom_closed_form():
    h, c, e = 0.5, 3.0, 1.0
    atoms = np.array([[2.25, 1.75, 2.0, 0.8]], dtype=np.float32)
    d = {"atoms": atoms, "natoms": 1, "h": h, "cutoff": c, "excl": e}
    pts = _lattice(11, 11, 11)
    v = T().cutcp_points(d, pts)
    p = pts.astype(np.float64) * h
    r = np.linalg.norm(p - atoms[0, :3].astype(np.float64), axis=1)
    ref = np.where(r < c, 0.8 / r * (1 - r * r / (c * c)) ** 2, 0.0)
    ref = np.where(r < e, 0.0, ref)
    assert np.allclose(v, ref, rtol=1e-6, atol=1e-12)  # fp32 inputs, fp64 terms
    assert np.count_nonzero(v) > 10 and np.count_nonzero(ref == 0) > 10


def test_cutcp_cutoff_boundary_is_zero():
    """An atom exactly at r = c contributes nothing (membership is r^2 < c^2,
    and the switch (1 - r^2/c^2)^2 vanishes there anyway)."""
    d = {"atoms": np.array([[3.0, 0.0, 0.0, 1.0]], dtype=np.float32), "natoms": 1,
         "h": 0.5, "cutoff": 3.0, "excl": 0.5}
    assert T().cutcp_points(d, np.array([[0, 0, 0]]))[0] == 0.0
    assert T().cutcp_points(d, np.array([[1, 0, 0]]))[0] > 0.0


def test_cutcp_mirror_charges_cancel():
    """+q and -q mirrored across the plane x = 8: V = 0 on that plane."""
    atoms = np.array([[5.5, 4.0, 4.25, 0.7], [10.5, 4.0, 4.25, -0.7]], dtype=np.float32)
    d = {"atoms": atoms, "natoms": 2, "h": 0.5, "cutoff": 6.0, "excl": 1.0}
    pts = _lattice(33, 17, 17)
    pts = pts[pts[:, 0] == 16]
    v = T().cutcp_points(d, pts)
    assert np.all(v == 0.0)


def test_cutcp_superposition_and_scaling():
    d = synth.preset("cutcp", "tiny", seed=2)
    a = d["atoms"]
    # keep only points far from every atom so no exclusion triggers
    pts = _lattice(d["nx"], d["ny"], d["nz"])
    p = pts.astype(np.float32) * np.float32(d["h"])
    dist2 = ((p[:, None, :] - a[None, :, :3]) ** 2).sum(-1).min(1)
    pts = pts[dist2 > 1.5]
    half = len(a) // 2
    da = dict(d, atoms=np.ascontiguousarray(a[:half]), natoms=half)
    db = dict(d, atoms=np.ascontiguousarray(a[half:]), natoms=len(a) - half)
    v = T().cutcp_points(d, pts)
    va = T().cutcp_points(da, pts)
    vb = T().cutcp_points(db, pts)
    assert np.allclose(v, va + vb, rtol=1e-12, atol=1e-12)
    a2 = a.copy()
    a2[:, 3] *= 2
    v2 = T().cutcp_points(dict(d, atoms=a2), pts)
    assert np.allclose(v2, 2 * v, rtol=1e-12, atol=1e-12)


def test_cutcp_full_lattice_matches_points():
    d = synth.preset("cutcp", "tiny", seed=1)
    full = T().cutcp(d)
    pts = _lattice(d["nx"], d["ny"], d["nz"])
    assert np.array_equal(full.ravel(), T().cutcp_points(d, pts))


def test_cutcp_binning_is_consistent():
    """The input layout (atoms sorted by cell, CSR offsets) lists every atom
    in the cell that contains it."""
    d = synth.preset("cutcp", "small", seed=4)
    n1 = d["ncell_1d"]
    cs = d["cell_start"]
    assert cs[0] == 0 and cs[-1] == d["natoms"]
    a = d["atoms"]
    for c in range(n1 ** 3):
        x, y, z = c % n1, (c // n1) % n1, c // (n1 * n1)
        blk = a[cs[c]:cs[c + 1], :3]
        lo = np.array([x, y, z], dtype=np.float32) * np.float32(d["cell"])
        assert np.all(blk >= lo) and np.all(blk < lo + np.float32(d["cell"]) + 1e-6)
    assert abs(a[:, 3].sum()) < 1e-2  # neutral molecules


# ---------------------------------------------------------------- tpacf
def _tpacf_numpy(d):
    """float32 numpy: elementwise products/sums round to nearest without FMA,
    same association as the definition; bins via np.searchsorted."""
    binb = d["binb"]
    asc = binb[::-1]
    nb = len(binb) + 1

    def hist(p, q, upper):
        dot = (p[0][:, None] * q[0][None, :] + p[1][:, None] * q[1][None, :]) + \
            p[2][:, None] * q[2][None, :]
        assert dot.dtype == np.float32
        if upper:
            iu = np.triu_indices(p.shape[1], k=1)
            dot = dot[iu]
        b = len(binb) - np.searchsorted(asc, dot.ravel(), side="right")
        return np.bincount(b, minlength=nb).astype(np.uint64)

    dd = hist(d["data"], d["data"], True)
    rr = sum(hist(r, r, True) for r in d["rand"])
    dr = sum(hist(d["data"], r, False) for r in d["rand"])
    return dd, rr, dr


def test_tpacf_numpy_float32():
    d = synth.preset("tpacf", "tiny")
    dd, rr, dr = T().tpacf(d)
    rdd, rrr, rdr = _tpacf_numpy(d)
    assert np.array_equal(dd, rdd) and np.array_equal(rr, rrr) and np.array_equal(dr, rdr)


def test_tpacf_pair_counts():
    d = synth.preset("tpacf", "small", seed=9)
    dd, rr, dr = T().tpacf(d)
    n, s = d["npts"], d["nsets"]
    assert dd.sum() == n * (n - 1) // 2
    assert rr.sum() == s * n * (n - 1) // 2
    assert dr.sum() == s * n * n


def test_tpacf_identical_points_in_bin0():
    """Coincident points (angle 0) land in the smallest-angle bin; antipodal
    points in the largest."""
    p = np.array([[1.0, 1.0, -1.0], [0.0, 0.0, 0.0], [0.0, 0.0, 0.0]], dtype=np.float32)
    d = {"data": p, "rand": p[None].copy(), "npts": 3, "nsets": 1, "binb": gen.tpacf_bin_edges()}
    dd, rr, dr = T().tpacf(d)
    assert dd[0] == 1 and dd[-1] == 2
    assert dr[0] == 5 and dr[-1] == 4


# ---------------------------------------------------------------- spmv
def test_spmv_scipy():
    from scipy.sparse import csr_matrix
    d = synth.preset("spmv", "small", seed=1)
    y = T().spmv(d)
    m = csr_matrix((d["val"].astype(np.float64), d["col"], d["row_ptr"]), shape=(d["n"], d["n"]))
    assert np.allclose(y, m @ d["x"].astype(np.float64), rtol=1e-13, atol=1e-13)
    assert d["nnz"] == (5 * 32 - 6) ** 2  # per axis sum_i #{di: 0 <= i+di < g} = 5g - 6


def test_spmv_identity():
    n = 50
    d = {"row_ptr": np.arange(n + 1, dtype=np.int32), "col": np.arange(n, dtype=np.int32),
         "val": np.ones(n, dtype=np.float32), "x": np.linspace(-3, 3, n).astype(np.float32), "n": n}
    assert np.array_equal(T().spmv(d), d["x"].astype(np.float64))


# ---------------------------------------------------------------- sgemm
def test_sgemm_numpy():
    d = synth.preset("sgemm", "tiny")
    c = T().sgemm(d)
    ref = d["a"].astype(np.float64) @ d["b"].astype(np.float64).T
    assert np.allclose(c, ref, rtol=1e-12, atol=1e-12)
    ij = np.array([[0, 0], [199, 135], [17, 3]])
    assert np.array_equal(T().sgemm_entries(d, ij), c[ij[:, 0], ij[:, 1]])


def test_sgemm_identity():
    k = 64
    a = synth.preset("sgemm", "tiny", k=k)["a"]
    d = {"a": a, "b": np.eye(k, dtype=np.float32), "m": a.shape[0], "n": k, "k": k}
    assert np.array_equal(T().sgemm(d), a.astype(np.float64))


# ---------------------------------------------------------------- mri-q
def test_mriq_phimag_float32():
    d = synth.preset("mriq", "tiny")
    pm = T().mriq_phimag(d)
    assert np.array_equal(pm, d["phir"] * d["phir"] + d["phii"] * d["phii"])


def test_mriq_complex_exponential():
    """Qr + i Qi = sum_k phiMag_k exp(2 pi i k.x) (numpy complex128)."""
    d = synth.preset("mriq", "tiny")
    pm, qr, qi = T().mriq(d)
    x = np.stack([d["x"], d["y"], d["z"]]).astype(np.float64)
    k = np.stack([d["kx"], d["ky"], d["kz"]]).astype(np.float64)
    q = np.exp(2j * np.pi * (k.T @ x)).T @ pm.astype(np.float64)
    assert np.allclose(qr, q.real, rtol=1e-10, atol=1e-10)
    assert np.allclose(qi, q.imag, rtol=1e-10, atol=1e-10)


def test_mriq_origin_and_dc():
    d = synth.preset("mriq", "tiny")
    d["x"][0] = d["y"][0] = d["z"][0] = 0.0
    d["kx"][5] = d["ky"][5] = d["kz"][5] = 0.0
    pm = T().mriq_phimag(d)
    qr, qi = T().mriq_points(d, np.array([0]))
    assert qr[0] == pytest.approx(pm.astype(np.float64).sum(), rel=1e-13)
    assert qi[0] == 0.0
    # numK = 1, sample at k = 0: every voxel sees Qr = phiMag, Qi = 0
    d1 = dict(d, numk=1, kx=d["kx"][5:6].copy(), ky=d["ky"][5:6].copy(), kz=d["kz"][5:6].copy(),
              phir=d["phir"][5:6].copy(), phii=d["phii"][5:6].copy())
    qr, qi = T().mriq_points(d1, np.arange(50))
    assert np.all(qr == np.float64(T().mriq_phimag(d1)[0])) and np.all(qi == 0.0)


# ---- sad (Parboil "sad") ----------------------------------

def _sad_numpy(d):
    """numpy brute force of the 4x4 SADs: the reference frame padded by edge
    replication (= clamping), every displacement sliced out at once."""
    w, h, R = d["w"], d["h"], d["R"]
    cur = d["cur"].astype(np.int64)
    ref = np.pad(d["ref"].astype(np.int64), R, mode="edge")
    side = 2 * R + 1
    out = np.empty((h // 16 * (w // 16), side * side, 16), dtype=np.int64)
    for p in range(side * side):
        dy, dx = p // side - R, p % side - R
        diff = np.abs(cur - ref[R + dy: R + dy + h, R + dx: R + dx + w])
        blk = diff.reshape(h // 4, 4, w // 4, 4).sum(axis=(1, 3))          # [h/4][w/4] 4x4 sums
        mbs = blk.reshape(h // 16, 4, w // 16, 4).transpose(0, 2, 1, 3)    # [my][mx][by][bx]
        out[:, p, :] = mbs.reshape(-1, 16)
    return out


def test_sad_matches_numpy_bruteforce():
    d = synth.preset("sad", "tiny", seed=3)
    s4, s8, s16 = T().sad(d)
    ref4 = _sad_numpy(d)
    assert np.array_equal(s4.astype(np.int64), ref4)
    # the 8x8 / 16x16 levels are the sums of the 4x4 SADs they cover
    q = ref4.reshape(ref4.shape[0], ref4.shape[1], 2, 2, 2, 2).sum(axis=(3, 5))   # [by2][bx2]
    assert np.array_equal(s8.astype(np.int64), q.reshape(ref4.shape[0], ref4.shape[1], 4))
    assert np.array_equal(s16.astype(np.int64), ref4.sum(axis=2))


def test_sad_identical_frames_zero_at_centre():
    d = synth.preset("sad", "tiny", seed=4)
    d = dict(d, ref=d["cur"].copy())
    s4, _, s16 = T().sad(d)
    centre = d["R"] * (2 * d["R"] + 1) + d["R"]
    assert not s4[:, centre, :].any() and not s16[:, centre].any()
    assert (s16[:, np.arange(s16.shape[1]) != centre] > 0).any()


def test_sad_global_shift_is_found():
    """ref = cur moved by (sx, sy) (no noise): every macroblock whose displaced
    block stays inside the frame has SAD 0 exactly at displacement (sx, sy)."""
    d = synth.preset("sad", "small", seed=5)
    sx, sy = 3, -2
    cur = d["cur"]
    ref = np.roll(np.roll(cur, sy, axis=0), sx, axis=1)   # ref[y+sy][x+sx] = cur[y][x]
    s4, s8, s16 = T().sad(dict(d, ref=np.ascontiguousarray(ref)))
    R, w, h = d["R"], d["w"], d["h"]
    p = (sy + R) * (2 * R + 1) + (sx + R)
    mbw = w // 16
    inside = [mb for mb in range(s16.shape[0])
              if 16 * (mb % mbw) + sx >= 0 and 16 * (mb % mbw) + 15 + sx < w and
              16 * (mb // mbw) + sy >= 0 and 16 * (mb // mbw) + 15 + sy < h]
    assert len(inside) > 50
    assert not s16[inside, p].any() and not s4[inside, p, :].any()


# ---- lbm (Parboil "lbm", D3Q19) ----------------------------

_LBM_C = np.array([[0, 0, 0], [1, 0, 0], [-1, 0, 0], [0, 1, 0], [0, -1, 0], [0, 0, 1], [0, 0, -1],
                   [1, 1, 0], [-1, -1, 0], [1, -1, 0], [-1, 1, 0], [1, 0, 1], [-1, 0, -1], [1, 0, -1],
                   [-1, 0, 1], [0, 1, 1], [0, -1, -1], [0, 1, -1], [0, -1, 1]])


def test_lbm_d3q19_lattice_properties():
    """The velocity set is D3Q19 with the textbook weights: sum w = 1,
    sum w c = 0, sum w c_a c_b = delta_ab / 3 (isotropy of the lattice)."""
    w = np.array([1 / 3] + [1 / 18] * 6 + [1 / 36] * 12)
    assert len({tuple(c) for c in _LBM_C}) == 19
    assert w.sum() == pytest.approx(1.0)
    assert np.allclose((w[:, None] * _LBM_C).sum(0), 0)
    assert np.allclose(np.einsum("q,qa,qb->ab", w, _LBM_C, _LBM_C), np.eye(3) / 3)


def test_lbm_conserves_mass_and_momentum():
    """BGK collision and periodic streaming conserve mass and (without
    obstacles) momentum; bounce-back conserves mass."""
    d = synth.preset("lbm", "tiny", seed=2)
    f0 = d["f0"].astype(np.float64)
    f = T().lbm(d)
    assert f.sum() == pytest.approx(f0.sum(), rel=1e-12)
    dn = dict(d, flags=np.zeros_like(d["flags"]))
    fn = T().lbm(dn)
    mom = lambda g: _LBM_C.astype(np.float64).T @ g.reshape(19, -1).sum(axis=1)  # noqa: E731
    assert np.allclose(mom(fn), mom(f0), rtol=0, atol=1e-9 * f0.sum())


def test_lbm_pure_streaming_is_a_shift():
    """omega = 0, no obstacles: one step moves every population by c_q."""
    d = synth.preset("lbm", "tiny", seed=3)
    d = dict(d, omega=0.0, steps=2, flags=np.zeros_like(d["flags"]))
    f = T().lbm(d)
    f0 = d["f0"].astype(np.float64)
    for q, (cx, cy, cz) in enumerate(_LBM_C):
        assert np.array_equal(f[q], np.roll(f0[q], (2 * cz, 2 * cy, 2 * cx), axis=(0, 1, 2)))


def test_lbm_uniform_equilibrium_is_a_fixed_point():
    d = synth.preset("lbm", "tiny", seed=4)
    w = np.array([1 / 3] + [1 / 18] * 6 + [1 / 36] * 12)
    rho, u = 1.02, np.array([0.03, -0.01, 0.02])
    cu = _LBM_C @ u
    feq = w * rho * (1 + 3 * cu + 4.5 * cu * cu - 1.5 * u @ u)
    f0 = np.broadcast_to(feq[:, None, None, None], d["f0"].shape).astype(np.float32).copy()
    f = T().lbm(dict(d, f0=f0, flags=np.zeros_like(d["flags"])))
    assert np.allclose(f, f0.astype(np.float64), rtol=1e-6, atol=0)


# ---- histo pipeline: prescan + intermediates (Parboil histo; f3) ------------

def test_histo_pipeline_numpy():
    d = synth.preset("histo_pipeline", "tiny", seed=6)
    lo, hi, bo, counts, sat = T().histo_pipeline(d)
    raw = d["raw"].astype(np.uint64)
    assert lo == raw.min() and hi == raw.max()
    ref = ((raw - lo) * d["bins"]) // (hi - lo + 1)
    assert np.array_equal(bo, ref.astype(np.uint32))
    assert np.array_equal(counts, np.bincount(ref, minlength=d["bins"]).astype(np.uint32))
    assert int(counts.sum()) == d["n"] and bo.max() < d["bins"]
    assert np.array_equal(sat, np.minimum(counts, 255).astype(np.uint8))


def test_histo_pipeline_recovers_the_bins():
    """raw = base + 4096 * s + U[0, 4096): when the extreme bins are both hit,
    the intermediates map (almost) every sample back to its generating bin s
    (lo and hi sit within one bin width of base and base + 4096 * bins, so
    only samples within that slack of a bin edge move)."""
    d = synth.preset("histo_pipeline", "small", seed=7)
    _, _, bo, _, _ = T().histo_pipeline(d)
    s = gen.gen_histo(d["n"], d["bins"], d["iters"], 4, 7)["samples"]
    if s.min() == 0 and s.max() == d["bins"] - 1:
        assert np.mean(bo == s) > 0.99 and np.all(np.abs(bo.astype(np.int64) - s) <= 1)


# ---- mri-gridding (Parboil) --------------------------------

def _gridding_numpy(d):
    """numpy brute force: every (grid point, sample) pair, the fp32 index
    decisions and products vectorised in float32, the sums in float64."""
    G, hw, lut = d["G"], np.float32(d["hw"]), d["lut"]
    ks = np.float32(len(lut) - 1) / hw
    g = np.zeros((G, G, G, 2))
    ax = np.arange(G, dtype=np.float32)
    for s in range(d["n"]):
        dx = np.abs(ax - d["x"][s]); dy = np.abs(ax - d["y"][s]); dz = np.abs(ax - d["z"][s])
        mx, my, mz = dx < hw, dy < hw, dz < hw
        if not (mx.any() and my.any() and mz.any()):
            continue
        wx = np.where(mx, lut[np.where(mx, (dx * ks).astype(np.int64), 0)], 0).astype(np.float32)
        wy = np.where(my, lut[np.where(my, (dy * ks).astype(np.int64), 0)], 0).astype(np.float32)
        wz = np.where(mz, lut[np.where(mz, (dz * ks).astype(np.int64), 0)], 0).astype(np.float32)
        w = (wy[:, None] * wx[None, :])[None, :, :] * wz[:, None, None]          # (wx*wy)*wz in fp32
        g[..., 0] += (w * d["re"][s]).astype(np.float64)
        g[..., 1] += (w * d["im"][s]).astype(np.float64)
    return g


def test_gridding_matches_numpy_bruteforce():
    d = synth.preset("gridding", "tiny", n=400, seed=2)
    assert np.allclose(T().gridding(d), _gridding_numpy(d), rtol=0, atol=1e-12)


def test_gridding_single_sample_closed_form():
    """One sample exactly on grid point (5, 6, 7) with value 1: the grid holds
    the separable table lut[(int)(|d| ks)]^3 around it, 0 elsewhere."""
    d = synth.preset("gridding", "tiny", seed=3)
    one = dict(d, n=1, x=np.array([5.0], np.float32), y=np.array([6.0], np.float32), z=np.array([7.0], np.float32),
               re=np.array([1.0], np.float32), im=np.array([0.0], np.float32))
    g = T().gridding(one)
    lut, hw = d["lut"], d["hw"]
    ks = np.float32(len(lut) - 1) / np.float32(hw)
    assert g[7, 6, 5, 0] == 1.0 and not g[..., 1].any()
    w1 = lut[int(np.float32(1.0) * ks)]
    assert g[7, 6, 6, 0] == pytest.approx(float(np.float32(np.float32(w1 * lut[0]) * lut[0])), rel=0)
    assert np.count_nonzero(g[..., 0]) == (2 * int(np.ceil(hw)) - 1) ** 3


def test_gridding_is_linear():
    d = synth.preset("gridding", "tiny", seed=4)
    h = d["n"] // 2
    part = lambda sl: dict(d, n=len(d["x"][sl]), **{k: np.ascontiguousarray(d[k][sl]) for k in ("x", "y", "z", "re", "im")})  # noqa: E731
    a, b = T().gridding(part(slice(0, h))), T().gridding(part(slice(h, None)))
    assert np.allclose(T().gridding(d), a + b, rtol=0, atol=1e-12)
