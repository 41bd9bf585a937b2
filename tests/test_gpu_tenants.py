"""GPU parity: every tenant through the C ABI, NATIVE and SHARED (persistent)
modes, against the CPU oracle -- bit-exact for integer work, within the north
star's 1e-4 (R-tol-1) for fp32 -- plus native == persistent bit-exact and the
per-VG coverage counters (every virtual group exactly once)."""
import numpy as np
import pytest

import synth
from tests.gpu_util import assert_close_fp32

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def acc():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no GPU")
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.runtime import Accel
    a = Accel(device=0, mode=abi.MODE_SHARED, verify=True)
    yield a
    a.close()


# small solver caps force few persistent CTAs -> many VGs per CTA
TINY_CAPS = (2, 2048, 65536, 233472, 32)


@pytest.fixture(scope="module")
def acc_tiny_caps():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no GPU")
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.runtime import Accel
    a = Accel(device=0, mode=abi.MODE_SHARED, verify=True, caps=abi.accel_caps(*TINY_CAPS))
    yield a
    a.close()


def run_modes(acc, job_factory):
    """Run the same job NATIVE then SHARED; return (native_result, shared_result, stats)."""
    from paper_conf_cgo_margiolaso16_b200 import abi
    out = {}
    st = {}
    for mode in (abi.MODE_NATIVE, abi.MODE_SHARED):
        acc.set_mode(mode)
        job = job_factory()
        s = acc.run([job])[0]
        assert s.coverage_ok == 1
        out[mode] = job.result()
        st[mode] = s
    acc.set_mode(abi.MODE_SHARED)
    return out[abi.MODE_NATIVE], out[abi.MODE_SHARED], st


def same(a: dict, b: dict):
    for k in a:
        assert np.array_equal(a[k], b[k]), k


# ---------------------------------------------------------------- mop
@pytest.mark.parametrize("nconst", [0, 1, 8, 11, 16, 36, 37])
def test_mop(acc_tiny_caps, oracle_lib, nconst):
    from paper_conf_cgo_margiolaso16_b200.jobs import MopJob
    d = synth.preset("mop", "tiny", nconst=nconst)
    nat, sh, st = run_modes(acc_tiny_caps, lambda: MopJob(d))
    ref = oracle_lib.mop(d)
    assert np.array_equal(nat["out"], ref)
    assert np.array_equal(sh["out"], ref)
    assert st[1].quota_initial < 37  # fewer persistent CTAs than VGs


def test_mop_small_fullcaps(acc, oracle_lib):
    from paper_conf_cgo_margiolaso16_b200.jobs import MopJob
    d = synth.preset("mop", "small")
    nat, sh, st = run_modes(acc, lambda: MopJob(d))
    ref = oracle_lib.mop(d)
    assert np.array_equal(nat["out"], ref) and np.array_equal(sh["out"], ref)


# ---------------------------------------------------------------- stencil
@pytest.mark.parametrize("size,over", [("tiny", {}), ("tiny", dict(nx=132, ny=9, nz=17, sweeps=2)),
                                       ("tiny", dict(nx=67, ny=13, nz=10, sweeps=3)),   # nx % 4 == 3
                                       ("tiny", dict(nx=129, ny=8, nz=9, sweeps=2)),    # one column past a tile
                                       ("tiny", dict(nx=2, ny=5, nz=4, sweeps=2)),      # all faces
                                       ("small", dict(sweeps=10))])
@pytest.mark.parametrize("kernel", ["default", "stencil_tma", "stencil", "stencil2", "stencil_z16"])
def test_stencil(acc_tiny_caps, oracle_lib, size, over, kernel):
    """default = the job's choice for this nx; "stencil" (8 rows per tile),
    "stencil2" (16 rows, two per warp) and "stencil_tma" (TMA ring) need
    nx % 4 == 0."""
    from paper_conf_cgo_margiolaso16_b200.jobs import StencilJob
    d = synth.preset("stencil", size, **over)
    if kernel != "default" and d["nx"] % 4:
        pytest.skip(f"{kernel} needs nx % 4 == 0")
    k = None if kernel == "default" else kernel
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: StencilJob(d, kernel=k))
    same(nat, sh)
    assert_close_fp32(sh["a"], oracle_lib.stencil(d), what="stencil")


@pytest.mark.parametrize("kernel", ["stencil_tma", "stencil", "stencil2", "stencil_z16"])
def test_stencil_default_sampled(acc, oracle_lib, kernel):
    """BASELINE size (512x512x64, 100 sweeps) in the bench's launch
    configuration; the oracle at full size is ~1.7e9 point-sweeps of plain C,
    so compare a handful of whole planes computed by the oracle on a z-slab
    that contains every point whose value can reach them (light cone)."""
    from paper_conf_cgo_margiolaso16_b200.jobs import StencilJob
    d = synth.preset("stencil", "default", sweeps=12)
    job = StencilJob(d, kernel=kernel)
    acc.run([job])
    got = job.result()["a"]
    # planes z in [20, 24): depend on z in [20-12, 24+12) only
    zlo, zhi, T = 8, 36, d["sweeps"]
    slab = dict(d, a0=np.ascontiguousarray(d["a0"][zlo:zhi]), nz=zhi - zlo)
    ref = oracle_lib.stencil(slab)
    assert_close_fp32(got[20:24], ref[20 - zlo:24 - zlo], what="stencil default")


# ---------------------------------------------------------------- histo
@pytest.mark.parametrize("size,over", [("tiny", {}), ("tiny", dict(bins=4096, sample_bytes=4)),
                                       ("tiny", dict(bins=16384, sample_bytes=4)),      # histo_wide
                                       ("tiny", dict(bins=10007, sample_bytes=4, iters=3)),  # odd bin count
                                       ("small", {}), ("small", dict(n=(1 << 18) + 13, iters=3))])
def test_histo(acc_tiny_caps, oracle_lib, size, over):
    from paper_conf_cgo_margiolaso16_b200.jobs import HistoJob
    d = synth.preset("histo", size, **over)
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: HistoJob(d))
    counts, sat = oracle_lib.histo(d)
    for r in (nat, sh):
        assert np.array_equal(r["counts"], counts)
        assert np.array_equal(r["sat"], sat)


def test_histo_default(acc, oracle_lib):
    """SURVEY §8(d).1 B200 default: 2^24 u32 samples, 16,384 bins (histo_wide)."""
    from paper_conf_cgo_margiolaso16_b200.jobs import HistoJob
    d = synth.preset("histo", "default", iters=3)
    assert d["n"] == 1 << 24 and d["bins"] == 16384
    nat, sh, _ = run_modes(acc, lambda: HistoJob(d))
    counts, sat = oracle_lib.histo(d)
    assert np.array_equal(sh["counts"], counts) and np.array_equal(nat["counts"], counts)
    assert np.array_equal(sh["sat"], sat) and np.array_equal(nat["sat"], sat)
    assert int(counts.sum()) == d["n"]


@pytest.mark.parametrize("per_vg", [8192, 32768, 61440])
def test_histo_wide_vg_sizes(acc_tiny_caps, oracle_lib, per_vg):
    """16-bit packed counters stay exact up to the largest allowed VG (the
    bins near the Gaussian peak take thousands of counts per VG)."""
    from paper_conf_cgo_margiolaso16_b200.jobs import HistoJob
    d = dict(synth.preset("histo", "small", bins=16384, sample_bytes=4, n=(1 << 19) + 77, iters=2), per_vg=per_vg)
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: HistoJob(d))
    counts, sat = oracle_lib.histo(d)
    for r in (nat, sh):
        assert np.array_equal(r["counts"], counts) and np.array_equal(r["sat"], sat)


# ---------------------------------------------------------------- mixes
def test_config1_mix_both_orders(acc, oracle_lib):
    """BASELINE config 1: stencil 64^3 + histo 256K u8, submitted together."""
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import HistoJob, StencilJob
    ds = synth.preset("stencil", "small", seed=1, sweeps=20)
    dh = synth.preset("histo", "small", seed=2)
    ref_s = oracle_lib.stencil(ds)
    ref_h = oracle_lib.histo(dh)
    for mode in (abi.MODE_NATIVE, abi.MODE_SHARED):
        acc.set_mode(mode)
        for order in ((0, 1), (1, 0)):
            jobs = [StencilJob(ds), HistoJob(dh)]
            st = acc.run([jobs[i] for i in order])
            assert all(s.coverage_ok == 1 for s in st)
            assert_close_fp32(jobs[0].result()["a"], ref_s)
            assert np.array_equal(jobs[1].result()["counts"], ref_h[0])
            if mode == abi.MODE_SHARED:
                # two concurrent requests share the device: quotas sum within it
                assert sum(s.quota_initial for s in st) <= 148 * 8
    acc.set_mode(abi.MODE_SHARED)


def test_e2e_host_buffers(acc, oracle_lib):
    """The request's own H2D/D2H copies (host pinned buffers) give the same result."""
    import torch
    from paper_conf_cgo_margiolaso16_b200.jobs import HistoJob
    d = synth.preset("histo", "small", seed=7)
    job = HistoJob(d)
    job.pin_host()
    job.inputs["samples"].zero_()  # the H2D copy must restore it
    torch.cuda.synchronize()
    acc.run([job], e2e=True)
    counts, _ = oracle_lib.histo(d)
    assert np.array_equal(job._pinned_out["counts"].numpy().view(np.uint32), counts)


def test_quota_matches_occupancy_for_single_tenant(acc):
    """K = 1: quota = min(G, SMs x cudaOccupancyMaxActiveBlocksPerMultiprocessor)."""
    import torch
    from paper_conf_cgo_margiolaso16_b200.jobs import StencilJob
    d = synth.preset("stencil", "default", sweeps=1)
    job = StencilJob(d)
    st = acc.run([job])[0]
    info = acc.kernel_info(job.kernel)
    sms = torch.cuda.get_device_properties(0).multi_processor_count
    g = int(np.prod(job.steps[0].grid))
    assert st.quota_initial == min(g, sms * info.occ_persistent)
    assert info.occ_persistent == info.occ_native


# ---------------------------------------------------------------- bfs
@pytest.mark.parametrize("size,over", [("tiny", {}), ("small", dict(seed=3)), ("small", dict(src=17, seed=5)),
                                       ("tiny", dict(deg_lo=0, deg_hi=2, seed=9))])
def test_bfs(acc_tiny_caps, oracle_lib, size, over):
    from paper_conf_cgo_margiolaso16_b200.jobs import BfsJob
    d = synth.preset("bfs", size, **over)
    ref, depth = oracle_lib.bfs(d)
    levels = depth + 3  # more launches than levels: empty frontiers must be no-ops
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: BfsJob(d, levels=levels))
    assert np.array_equal(nat["level"], ref)
    assert np.array_equal(sh["level"], ref)


def test_bfs_default(acc, oracle_lib):
    from paper_conf_cgo_margiolaso16_b200.jobs import BfsJob
    d = synth.preset("bfs", "default")
    ref, depth = oracle_lib.bfs(d)
    assert depth + 1 < 24  # the bench's launch count covers every level
    nat, sh, _ = run_modes(acc, lambda: BfsJob(d))
    assert np.array_equal(nat["level"], ref) and np.array_equal(sh["level"], ref)


# ---------------------------------------------------------------- cutcp
# default 1-A cells: ~290 cell rows per VG, three gather batches of 128 rows;
# 4-A and 2-A cells: one batch, longer rows (the row gather, cutcp.cuh)
@pytest.mark.parametrize("size,over", [("tiny", {}), ("tiny", dict(seed=5, box=24.0)), ("small", {}),
                                       ("tiny", dict(cell=4.0)), ("small", dict(seed=2, cell=2.0))])
def test_cutcp(acc_tiny_caps, oracle_lib, size, over):
    from paper_conf_cgo_margiolaso16_b200.jobs import CutcpJob
    d = synth.preset("cutcp", size, **over)
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: CutcpJob(d))
    same(nat, sh)
    ref = oracle_lib.cutcp(d)
    assert np.array_equal(sh["v"] == 0, ref == 0)  # exclusion decided identically
    assert_close_fp32(sh["v"], ref, what="cutcp")


def test_cutcp_default_sampled(acc, oracle_lib):
    from paper_conf_cgo_margiolaso16_b200.jobs import CutcpJob
    d = synth.preset("cutcp", "default")
    job = CutcpJob(d)
    acc.run([job])
    v = job.result()["v"]
    r = np.random.Generator(np.random.PCG64(1))
    ijk = np.stack([r.integers(0, d["nx"], 3000), r.integers(0, d["ny"], 3000), r.integers(0, d["nz"], 3000)], 1)
    ref = oracle_lib.cutcp_points(d, ijk)
    got = v[ijk[:, 2], ijk[:, 1], ijk[:, 0]]
    assert np.array_equal(got == 0, ref == 0)
    assert_close_fp32(got, ref, what="cutcp default")


# ---------------------------------------------------------------- tpacf
@pytest.mark.parametrize("size,over", [("tiny", {}), ("small", {}), ("tiny", dict(npts=257, nsets=2))])
def test_tpacf(acc_tiny_caps, oracle_lib, size, over):
    from paper_conf_cgo_margiolaso16_b200.jobs import TpacfJob
    d = synth.preset("tpacf", size, **over)
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: TpacfJob(d))
    dd, rr, dr = oracle_lib.tpacf(d)
    for r in (nat, sh):
        assert np.array_equal(r["dd"], dd) and np.array_equal(r["rr"], rr) and np.array_equal(r["dr"], dr)


def test_tpacf_default(acc, oracle_lib):
    from paper_conf_cgo_margiolaso16_b200.jobs import TpacfJob
    d = synth.preset("tpacf", "default")
    job = TpacfJob(d)
    acc.run([job])
    dd, rr, dr = oracle_lib.tpacf(d)
    r = job.result()
    assert np.array_equal(r["dd"], dd) and np.array_equal(r["rr"], rr) and np.array_equal(r["dr"], dr)


# ---------------------------------------------------------------- config 2
def test_config2_fig2_mix(acc, oracle_lib):
    """Fig. 2 mix (bfs + cutcp + stencil + tpacf) at bench sizes, both modes:
    outputs under concurrency equal the isolated oracle results."""
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import make_job
    names = ["bfs", "cutcp", "stencil", "tpacf"]
    ds = {"bfs": synth.preset("bfs", "default", seed=3),
          "cutcp": synth.preset("cutcp", "small", seed=4),
          "stencil": synth.preset("stencil", "small", seed=5, sweeps=10),
          "tpacf": synth.preset("tpacf", "small", seed=6)}
    refs = {"bfs": oracle_lib.bfs(ds["bfs"])[0], "cutcp": oracle_lib.cutcp(ds["cutcp"]),
            "stencil": oracle_lib.stencil(ds["stencil"]), "tpacf": oracle_lib.tpacf(ds["tpacf"])}
    for mode in (abi.MODE_SHARED, abi.MODE_NATIVE):
        acc.set_mode(mode)
        jobs = [make_job(n, ds[n]) for n in names]
        st = acc.run(jobs)
        assert all(s.coverage_ok == 1 for s in st)
        assert np.array_equal(jobs[0].result()["level"], refs["bfs"])
        assert_close_fp32(jobs[1].result()["v"], refs["cutcp"])
        assert_close_fp32(jobs[2].result()["a"], refs["stencil"])
        r = jobs[3].result()
        assert np.array_equal(r["dd"], refs["tpacf"][0]) and np.array_equal(r["dr"], refs["tpacf"][2])
        if mode == abi.MODE_SHARED:
            assert len({s.quota_initial for s in st}) >= 1
    acc.set_mode(abi.MODE_SHARED)


def _stencil_fp32_replica(d):
    """numpy float32 with the kernels' association ("numpy
    float32 with the same parenthesisation reproduces the result exactly"):
    ((((((zm + zp) + ym) + yp) + xm) + xp) * c1) - (a * c0), faces copy."""
    a = d["a0"].reshape(d["nz"], d["ny"], d["nx"]).astype(np.float32)
    c0, c1 = np.float32(d["c0"]), np.float32(d["c1"])
    for _ in range(d["sweeps"]):
        o = a.copy()
        s = a[:-2, 1:-1, 1:-1] + a[2:, 1:-1, 1:-1]
        s = s + a[1:-1, :-2, 1:-1]
        s = s + a[1:-1, 2:, 1:-1]
        s = s + a[1:-1, 1:-1, :-2]
        s = s + a[1:-1, 1:-1, 2:]
        o[1:-1, 1:-1, 1:-1] = s * c1 - a[1:-1, 1:-1, 1:-1] * c0
        a = o
    return a


@pytest.mark.parametrize("kernel,over", [("stencil_tma", dict(nx=136, ny=17, nz=19, sweeps=4)),
                                         ("stencil_bulk", dict(nx=136, ny=17, nz=19, sweeps=4)),
                                         ("stencil_bulk", dict(nx=260, ny=9, nz=8, sweeps=3)),
                                         ("stencil", dict(nx=136, ny=17, nz=19, sweeps=4)),
                                         ("stencil2", dict(nx=136, ny=17, nz=19, sweeps=4)),
                                         ("stencil2", dict(nx=260, ny=33, nz=8, sweeps=3)),
                                         ("stencil2", dict(nx=4, ny=3, nz=3, sweeps=2)),
                                         ("stencil_z16", dict(nx=136, ny=17, nz=37, sweeps=4)),
                                         ("stencil_z16", dict(nx=132, ny=9, nz=16, sweeps=3)),
                                         ("stencil_x", dict(nx=70, ny=21, nz=19, sweeps=3))])
def test_stencil_bit_exact_fp32_sequence(acc_tiny_caps, kernel, over):
    """Every stencil kernel computes the pinned fp32 round-to-nearest sequence
    (no FMA contraction), so native, persistent and a numpy float32 replica
    agree bit for bit."""
    from paper_conf_cgo_margiolaso16_b200.jobs import StencilJob
    d = synth.preset("stencil", "tiny", **over)
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: StencilJob(d, kernel=kernel))
    ref = _stencil_fp32_replica(d)
    assert np.array_equal(nat["a"], ref) and np.array_equal(sh["a"], ref)


@pytest.mark.parametrize("qsplit", [1, 3, 7])
def test_tpacf_qsplit(acc_tiny_caps, oracle_lib, qsplit):
    """VGs over parts of the other set's tiles (any split, including more
    parts than a DD/RR block has tiles) count every pair exactly once."""
    from paper_conf_cgo_margiolaso16_b200.jobs import TpacfJob
    d = dict(synth.preset("tpacf", "small", seed=8), qsplit=qsplit)
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: TpacfJob(d))
    dd, rr, dr = oracle_lib.tpacf(d)
    for r in (nat, sh):
        assert np.array_equal(r["dd"], dd) and np.array_equal(r["rr"], rr) and np.array_equal(r["dr"], dr)


@pytest.mark.parametrize("size", ["tiny", "small"])
def test_histo_pipeline(acc_tiny_caps, oracle_lib, size):
    """Parboil histo's full pipeline (f3): prescan range and intermediate bin
    stream, then the histogram -- bit-exact in both modes."""
    from paper_conf_cgo_margiolaso16_b200.jobs import HistoPipelineJob
    d = synth.preset("histo_pipeline", size)
    lo, hi, bo, counts, sat = oracle_lib.histo_pipeline(d)
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: HistoPipelineJob(d))
    for r in (nat, sh):
        assert (r["lo"], r["hi"]) == (lo, hi)
        assert np.array_equal(r["counts"], counts) and np.array_equal(r["sat"], sat)


def test_histo_pipeline_default(acc, oracle_lib):
    from paper_conf_cgo_margiolaso16_b200.jobs import HistoPipelineJob
    d = synth.preset("histo_pipeline", "default", iters=3)
    lo, hi, bo, counts, sat = oracle_lib.histo_pipeline(d)
    nat, sh, _ = run_modes(acc, lambda: HistoPipelineJob(d))
    for r in (nat, sh):
        assert (r["lo"], r["hi"]) == (lo, hi) and np.array_equal(r["counts"], counts)


@pytest.mark.parametrize("edges", ["linear", "near_one"])
def test_tpacf_custom_edges(acc_tiny_caps, oracle_lib, edges):
    """Bin edges the exponent table cannot separate (many edges in one octave
    of 1 - d: the binary-search fallback) and edges crowding d = 1: still
    bit-exact against the oracle."""
    from paper_conf_cgo_margiolaso16_b200.jobs import TpacfJob
    d = synth.preset("tpacf", "tiny", seed=12)
    if edges == "linear":
        b = np.linspace(0.99, -0.9, 21)
    else:
        b = 1.0 - np.geomspace(1e-7, 1.5, 21)
    d = dict(d, binb=np.ascontiguousarray(np.sort(b)[::-1].astype(np.float32)))
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: TpacfJob(d))
    dd, rr, dr = oracle_lib.tpacf(d)
    for r in (nat, sh):
        assert np.array_equal(r["dd"], dd) and np.array_equal(r["rr"], rr) and np.array_equal(r["dr"], dr)


@pytest.mark.parametrize("kernel", ["stencil_tma", "stencil_bulk"])
def test_stencil_async_staging_next_to_bfs(acc, kernel):
    """Regression for the ring-slot race (stencil staging): a
    consumer warp released a slot before its ld.shared had read it, and next
    to bfs (whose shared-memory atomics slow those loads) the producer's TMA of
    a later plane landed first.  The TMA/bulk-staged sweep must equal the
    cp.async sweep bit for bit (same pinned fp32 op sequence) at the bench's
    size, next to bfs, in every mode."""
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import StencilJob, make_job
    d = synth.preset("stencil", "default", sweeps=12)
    acc.set_mode(abi.MODE_NATIVE, abi.POLICY_STATIC)
    ref_job = StencilJob(d, kernel="stencil")
    acc.run([ref_job])
    ref = ref_job.result()["a"]
    bfs = make_job("bfs", synth.preset("bfs", "default"))
    bfs.fit_levels(acc)
    try:
        for mode, pol in [(abi.MODE_NATIVE, abi.POLICY_STATIC), (abi.MODE_SHARED, abi.POLICY_STATIC),
                          (abi.MODE_SHARED, abi.POLICY_RESOLVE)]:
            acc.set_mode(mode, pol)
            for _ in range(2):
                sj = StencilJob(d, kernel=kernel)
                acc.run([bfs, sj])
                got = sj.result()["a"]
                assert np.array_equal(got, ref), (mode, pol, int((got != ref).sum()))
    finally:
        acc.set_mode(abi.MODE_SHARED, abi.POLICY_STATIC)
