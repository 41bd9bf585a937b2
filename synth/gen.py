"""Seeded generators for the tenant inputs (numpy PCG64, explicit seeds).

Every generator returns a plain dict of numpy arrays and python scalars.  The
dict is the *input* of a tenant; outputs are never produced here.
"""
from __future__ import annotations

import math

import numpy as np

__all__ = [
    "rng",
    "gen_mop",
    "gen_stencil",
    "gen_histo",
    "gen_bfs",
    "gen_cutcp",
    "gen_tpacf",
    "gen_spmv",
    "gen_sgemm",
    "gen_mriq",
    "gen_sad",
    "gen_lbm",
    "gen_histo_raw",
    "gen_gridding",
    "GENERATORS",
]


def rng(seed: int) -> np.random.Generator:
    return np.random.Generator(np.random.PCG64(seed))


def gen_mop(n: int, block: int = 256, nconst: int | None = None, seed: int = 0) -> dict:
    """Fig. 8a example kernel inputs: two fp32 buffers."""
    r = rng(seed)
    if nconst is None:
        nconst = (n // block) // 2
    return {
        "ina": r.uniform(-1.0, 1.0, n).astype(np.float32),
        "inb": r.uniform(-1.0, 1.0, n).astype(np.float32),
        "n": int(n),
        "block": int(block),
        "nconst": int(nconst),
    }


def gen_stencil(nx: int, ny: int, nz: int, sweeps: int, seed: int = 0) -> dict:
    """7-point Jacobi input field A0[nz][ny][nx] ~ U[0,1) (x fastest)."""
    r = rng(seed)
    c0 = np.float32(1.0) / np.float32(6.0)
    c1 = c0 / np.float32(6.0)
    return {
        "a0": r.random((nz, ny, nx), dtype=np.float32),
        "nx": int(nx), "ny": int(ny), "nz": int(nz),
        "sweeps": int(sweeps),
        "c0": float(c0), "c1": float(c1),
    }


def gen_histo(n: int, bins: int, iters: int, sample_bytes: int = 4, seed: int = 0) -> dict:
    """Skewed samples in [0, bins): 70 % discretised Gaussian (sigma = bins/64,
    mean bins/2), 30 % uniform.  u8 samples require bins == 256."""
    r = rng(seed)
    if sample_bytes == 1 and bins != 256:
        raise ValueError("u8 samples need 256 bins")
    k = int(round(0.7 * n))
    g = np.rint(r.normal(bins / 2.0, bins / 64.0, k))
    g = np.clip(g, 0, bins - 1)
    u = r.integers(0, bins, n - k)
    s = np.concatenate([g, u])
    r.shuffle(s)
    dt = np.uint8 if sample_bytes == 1 else np.uint32
    return {"samples": s.astype(dt), "n": int(n), "bins": int(bins),
            "iters": int(iters), "sample_bytes": int(sample_bytes)}


def gen_bfs(nv: int, deg_lo: int = 1, deg_hi: int = 11, src: int = 0, seed: int = 0) -> dict:
    """Directed random graph in CSR: out-degree ~ U{deg_lo..deg_hi}, uniform
    targets (self loops and duplicate edges allowed, as in a raw edge list)."""
    r = rng(seed)
    deg = r.integers(deg_lo, deg_hi + 1, nv)
    row_ptr = np.zeros(nv + 1, dtype=np.int64)
    np.cumsum(deg, out=row_ptr[1:])
    ne = int(row_ptr[-1])
    col = r.integers(0, nv, ne).astype(np.int32)
    if ne >= 2**31:
        raise ValueError("too many edges")
    return {"row_ptr": row_ptr.astype(np.uint32), "col": col, "nv": int(nv),
            "ne": ne, "src": int(src)}


def gen_cutcp(box: float, density: float = 0.1, h: float = 0.5, cutoff: float = 12.0,
              excl: float = 1.0, cell: float = 4.0, seed: int = 0) -> dict:
    """Water-like charges in a cubic box [0, box)^3.

    Molecules = O(-0.834) at a uniform position plus two H(+0.417) at a ~1 A
    offset (wrapped into the box).  Atoms are stored as float4 (x, y, z, q),
    sorted into a uniform grid of `cell`-A cells (x fastest) with CSR offsets
    `cell_start` -- an input layout, like Parboil's host-side binning.  The
    workload keeps 4-A cells; 1-A cells make cutcp 25 % faster alone but
    change the C2 mix's balance (cutcp cell size).
    Lattice point (i, j, k) sits at h*(i, j, k), i in [0, box/h].
    """
    r = rng(seed)
    ncell_1d = int(round(box / cell))
    if abs(ncell_1d * cell - box) > 1e-6:
        raise ValueError("box must be a multiple of the cell size")
    nmol = int(round(box ** 3 * density / 3.0))
    o = r.uniform(0.0, box, (nmol, 3))
    d1 = r.normal(0.0, 1.0, (nmol, 3))
    d1 /= np.linalg.norm(d1, axis=1, keepdims=True)
    d2 = r.normal(0.0, 1.0, (nmol, 3))
    d2 /= np.linalg.norm(d2, axis=1, keepdims=True)
    pos = np.concatenate([o, o + 0.9572 * d1, o + 0.9572 * d2])
    pos = np.mod(pos, box)
    q = np.concatenate([np.full(nmol, -0.834), np.full(nmol, 0.417), np.full(nmol, 0.417)])
    pos32 = pos.astype(np.float32)
    pos32 = np.minimum(pos32, np.nextafter(np.float32(box), np.float32(0)))
    cidx = np.minimum((pos32 / np.float32(cell)).astype(np.int64), ncell_1d - 1)
    cid = cidx[:, 0] + ncell_1d * (cidx[:, 1] + ncell_1d * cidx[:, 2])
    order = np.argsort(cid, kind="stable")
    atoms = np.empty((len(q), 4), dtype=np.float32)
    atoms[:, :3] = pos32[order]
    atoms[:, 3] = q[order].astype(np.float32)
    ncell = ncell_1d ** 3
    counts = np.bincount(cid, minlength=ncell)
    cell_start = np.zeros(ncell + 1, dtype=np.int32)
    np.cumsum(counts, out=cell_start[1:])
    nl = int(round(box / h)) + 1
    return {
        "atoms": atoms, "natoms": int(len(q)), "cell_start": cell_start,
        "ncell_1d": ncell_1d, "cell": float(cell), "box": float(box),
        "nx": nl, "ny": nl, "nz": nl, "h": float(h), "cutoff": float(cutoff),
        "excl": float(excl),
    }


def tpacf_bin_edges(nbins: int = 20, min_arcmin: float = 1.0, bins_per_dec: int = 5) -> np.ndarray:
    """binb[k] = cos(10^(k/5) arcmin), k = 0..20 (descending), computed in fp64
    and rounded to fp32.  An input of the tenant, like Parboil's binb array."""
    k = np.arange(nbins + 1, dtype=np.float64)
    arcmin = min_arcmin * 10.0 ** (k / bins_per_dec)
    return np.cos(arcmin / 60.0 * math.pi / 180.0).astype(np.float32)


def _sphere(r: np.random.Generator, n: int) -> np.ndarray:
    v = r.normal(0.0, 1.0, (n, 3))
    v /= np.linalg.norm(v, axis=1, keepdims=True)
    return np.ascontiguousarray(v.T.astype(np.float32))  # SoA [3][n]


def gen_tpacf(npts: int, nsets: int, seed: int = 0) -> dict:
    """Data and `nsets` random catalogues of unit vectors, SoA layout
    data[3][npts], rand[nsets][3][npts]."""
    r = rng(seed)
    data = _sphere(r, npts)
    rand = np.stack([_sphere(r, npts) for _ in range(nsets)])
    return {"data": data, "rand": rand, "npts": int(npts), "nsets": int(nsets),
            "binb": tpacf_bin_edges()}


def gen_spmv(grid: int, reach: int = 2, iters: int = 1, seed: int = 0) -> dict:
    """CSR matrix of a grid x grid lattice with (2*reach+1)^2 coupling
    (Dubcova-like), values and x ~ U[-1, 1)."""
    r = rng(seed)
    n = grid * grid
    ii, jj = np.meshgrid(np.arange(grid), np.arange(grid), indexing="ij")
    ii = ii.ravel()
    jj = jj.ravel()
    cols = []
    for di in range(-reach, reach + 1):
        for dj in range(-reach, reach + 1):
            ni, nj = ii + di, jj + dj
            ok = (ni >= 0) & (ni < grid) & (nj >= 0) & (nj < grid)
            c = np.where(ok, ni * grid + nj, -1)
            cols.append(c)
    cols = np.stack(cols, axis=1)  # [n][25], row-major neighbours in sorted order
    mask = cols >= 0
    nnz_row = mask.sum(axis=1)
    row_ptr = np.zeros(n + 1, dtype=np.int32)
    np.cumsum(nnz_row, out=row_ptr[1:])
    col = cols[mask].astype(np.int32)
    val = r.uniform(-1.0, 1.0, len(col)).astype(np.float32)
    x = r.uniform(-1.0, 1.0, n).astype(np.float32)
    return {"row_ptr": row_ptr, "col": col, "val": val, "x": x, "n": int(n),
            "nnz": int(len(col)), "iters": int(iters)}


def gen_sgemm(m: int, n: int, k: int, seed: int = 0) -> dict:
    """A[m][k], B[n][k] (both K-major) ~ U[-1, 1); C = A B^T."""
    r = rng(seed)
    return {"a": r.uniform(-1.0, 1.0, (m, k)).astype(np.float32),
            "b": r.uniform(-1.0, 1.0, (n, k)).astype(np.float32),
            "m": int(m), "n": int(n), "k": int(k)}


def gen_mriq(nvox_1d: int, numk: int, seed: int = 0) -> dict:
    """Voxel centres on a half-integer grid (i - n/2 + 0.5), k-space samples
    k ~ U[-0.5, 0.5)^3, phi ~ U[-1, 1) (SoA)."""
    r = rng(seed)
    c = (np.arange(nvox_1d, dtype=np.float64) - nvox_1d / 2 + 0.5)
    zz, yy, xx = np.meshgrid(c, c, c, indexing="ij")
    return {
        "x": xx.ravel().astype(np.float32), "y": yy.ravel().astype(np.float32),
        "z": zz.ravel().astype(np.float32),
        "kx": r.uniform(-0.5, 0.5, numk).astype(np.float32),
        "ky": r.uniform(-0.5, 0.5, numk).astype(np.float32),
        "kz": r.uniform(-0.5, 0.5, numk).astype(np.float32),
        "phir": r.uniform(-1.0, 1.0, numk).astype(np.float32),
        "phii": r.uniform(-1.0, 1.0, numk).astype(np.float32),
        "numx": int(nvox_1d ** 3), "numk": int(numk),
    }


def gen_sad(w: int, h: int, R: int = 16, seed: int = 0) -> dict:
    """Two video frames (u16 pixels < 256): a smooth random field (sum of
    Gaussian-blurred noise octaves) and the same field moved by a seeded
    global shift plus noise -- motion-estimation-shaped input [ext Parboil sad]."""
    r = rng(seed)
    base = np.zeros((h + 64, w + 64))
    for sc in (1, 4, 16):
        nz = r.normal(0.0, 1.0, ((h + 64) // sc + 2, (w + 64) // sc + 2))
        up = np.kron(nz, np.ones((sc, sc)))[: h + 64, : w + 64]
        base += up * sc
    base = (base - base.min()) / (base.max() - base.min()) * 255.0
    sy, sx = (int(v) for v in r.integers(-6, 7, 2))
    cur = base[32: 32 + h, 32: 32 + w]
    ref = base[32 + sy: 32 + sy + h, 32 + sx: 32 + sx + w] + r.normal(0.0, 3.0, (h, w))
    q = lambda a: np.clip(np.rint(a), 0, 255).astype(np.uint16)  # noqa: E731
    return {"cur": np.ascontiguousarray(q(cur)), "ref": np.ascontiguousarray(q(ref)),
            "w": int(w), "h": int(h), "R": int(R)}


def gen_lbm(nx: int, ny: int, nz: int, steps: int, omega: float = 1.95, seed: int = 0) -> dict:
    """D3Q19 lattice (SoA f[q][z][y][x] fp32) near equilibrium: rho = 1 +- 1 %,
    u ~ U[-0.05, 0.05)^3 per cell, f = feq(rho, u) + 1e-3 w_q noise; obstacles
    = a few seeded spheres (~5 % of the cells) [ext Parboil lbm: its obstacle
    file is not available]."""
    r = rng(seed)
    c = np.array([[0, 0, 0], [1, 0, 0], [-1, 0, 0], [0, 1, 0], [0, -1, 0], [0, 0, 1], [0, 0, -1],
                  [1, 1, 0], [-1, -1, 0], [1, -1, 0], [-1, 1, 0], [1, 0, 1], [-1, 0, -1], [1, 0, -1],
                  [-1, 0, 1], [0, 1, 1], [0, -1, -1], [0, 1, -1], [0, -1, 1]], dtype=np.float64)
    w = np.array([1 / 3] + [1 / 18] * 6 + [1 / 36] * 12)
    shape = (nz, ny, nx)
    rho = 1.0 + 0.01 * r.uniform(-1, 1, shape)
    u = 0.05 * r.uniform(-1, 1, (3,) + shape)
    cu = np.einsum("qd,d...->q...", c, u)
    uu = (u * u).sum(0)
    f = w[:, None, None, None] * rho * (1 + 3 * cu + 4.5 * cu * cu - 1.5 * uu)
    f += 1e-3 * w[:, None, None, None] * r.uniform(-1, 1, f.shape)
    zz, yy, xx = np.meshgrid(np.arange(nz), np.arange(ny), np.arange(nx), indexing="ij")
    flags = np.zeros(shape, dtype=np.uint8)
    for _ in range(max(1, (nx * ny * nz) // 40000)):
        cz, cy, cx = r.uniform(0, nz), r.uniform(0, ny), r.uniform(0, nx)
        rad = r.uniform(2.0, max(2.5, min(nx, ny, nz) / 8))
        flags |= (((zz - cz) ** 2 + (yy - cy) ** 2 + (xx - cx) ** 2) < rad * rad).astype(np.uint8)
    return {"f0": np.ascontiguousarray(f.astype(np.float32)), "flags": np.ascontiguousarray(flags),
            "nx": int(nx), "ny": int(ny), "nz": int(nz), "steps": int(steps), "omega": float(omega)}


def gen_histo_raw(n: int, bins: int, iters: int, seed: int = 0) -> dict:
    """Raw u32 samples for Parboil histo's full pipeline: the skewed bin
    distribution of gen_histo, scaled by 4096, plus a uniform in-bin offset
    and a seeded base (the prescan finds the range, the intermediates map it
    back to bins)."""
    r = rng(seed)
    s = gen_histo(n, bins, iters, 4, seed)["samples"].astype(np.uint64)
    base = int(r.integers(1_000, 1_000_000))
    raw = base + s * 4096 + r.integers(0, 4096, n, dtype=np.uint64)
    return {"raw": np.ascontiguousarray(raw.astype(np.uint32)), "n": int(n), "bins": int(bins), "iters": int(iters)}


def gen_gridding(G: int, n: int, W: float = 4.0, L: int = 1024, seed: int = 0) -> dict:
    """MRI k-space samples for gridding [ext Parboil mri-gridding]: half
    uniform in [0, G)^3, half on 64 jittered radial spokes (a radial
    acquisition's lines), complex values U[-1, 1)^2; the
    separable Kaiser-Bessel kernel of width W (half-width W/2) tabulated at L
    points, beta = pi sqrt((W/2)^2 (2 - 0.5)^2 - 0.8) (oversampling 2),
    normalised to 1 at distance 0 -- computed here in fp64."""
    r = rng(seed)
    hw = W / 2.0
    c = G / 2.0
    # half the samples uniform in the volume, half on 64 jittered radial
    # spokes with radius pdf ~ r^2 (each spoke's samples spread like a ball's
    # volume: no 1/r^2 pile-up at the centre that would leave one gridding
    # tile with 50x the average work)
    nu = n // 2
    t = np.cbrt(r.uniform(0, 1, n - nu)) * r.choice([-1.0, 1.0], n - nu)
    dirs = r.normal(0, 1, (64, 3))
    dirs /= np.linalg.norm(dirs, axis=1, keepdims=True)
    pick = dirs[r.integers(0, 64, n - nu)]
    spokes = c + (G / 2.0 - hw) * t[:, None] * pick + r.normal(0, 1.0, (n - nu, 3))
    pts = np.concatenate([r.uniform(0, G, (nu, 3)), spokes])
    pts = np.clip(pts, 0.0, np.nextafter(G, 0))
    beta = np.pi * np.sqrt((W / 2.0) ** 2 * (2.0 - 0.5) ** 2 - 0.8)
    dist = np.arange(L) * hw / (L - 1)
    arg = beta * np.sqrt(np.maximum(0.0, 1.0 - (dist / hw) ** 2))
    lut = np.i0(arg) / np.i0(beta)
    return {"x": np.ascontiguousarray(pts[:, 0].astype(np.float32)), "y": np.ascontiguousarray(pts[:, 1].astype(np.float32)),
            "z": np.ascontiguousarray(pts[:, 2].astype(np.float32)),
            "re": r.uniform(-1, 1, n).astype(np.float32), "im": r.uniform(-1, 1, n).astype(np.float32),
            "lut": lut.astype(np.float32), "n": int(n), "G": int(G), "hw": float(hw)}


GENERATORS = {
    "mop": gen_mop, "stencil": gen_stencil, "histo": gen_histo, "bfs": gen_bfs,
    "cutcp": gen_cutcp, "tpacf": gen_tpacf, "spmv": gen_spmv, "sgemm": gen_sgemm,
    "mriq": gen_mriq, "sad": gen_sad, "lbm": gen_lbm, "histo_pipeline": gen_histo_raw,
    "gridding": gen_gridding,
}
