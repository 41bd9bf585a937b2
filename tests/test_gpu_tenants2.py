"""GPU parity for spmv, sgemm and mri-q (both modes, coverage, oracle)."""
import numpy as np
import pytest

import synth
from tests.gpu_util import assert_close_fp32
from tests.test_gpu_tenants import acc, acc_tiny_caps, run_modes, same  # noqa: F401  (fixtures)

pytestmark = pytest.mark.gpu


@pytest.mark.parametrize("size,over", [("tiny", {}), ("small", dict(iters=3)), ("tiny", dict(grid=7, reach=3)),
                                       ("tiny", dict(grid=5, reach=1))])
@pytest.mark.parametrize("kernel", ["spmv", "spmv_v4"])
def test_spmv(acc_tiny_caps, oracle_lib, size, over, kernel):
    """spmv_v4: 128-bit chunk loads over padded col/val (any nnz % 4)."""
    from paper_conf_cgo_margiolaso16_b200.jobs import SpmvJob
    d = synth.preset("spmv", size, **over)
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: SpmvJob(d, kernel=kernel))
    same(nat, sh)
    assert_close_fp32(sh["y"], oracle_lib.spmv(d), what="spmv")


@pytest.mark.parametrize("kernel", ["spmv", "spmv_v4"])
def test_spmv_default(acc, oracle_lib, kernel):
    from paper_conf_cgo_margiolaso16_b200.jobs import SpmvJob
    d = synth.preset("spmv", "default", iters=2)
    nat, sh, _ = run_modes(acc, lambda: SpmvJob(d, kernel=kernel))
    same(nat, sh)
    assert_close_fp32(sh["y"], oracle_lib.spmv(d), what="spmv default")


@pytest.mark.parametrize("size,over", [("tiny", {}), ("small", {}), ("tiny", dict(m=129, n=257, k=36))])
def test_sgemm(acc_tiny_caps, oracle_lib, size, over):
    from paper_conf_cgo_margiolaso16_b200.jobs import SgemmJob
    d = synth.preset("sgemm", size, **over)
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: SgemmJob(d))
    same(nat, sh)
    assert_close_fp32(sh["c"], oracle_lib.sgemm(d), what="sgemm")


def test_sgemm_default_sampled(acc, oracle_lib):
    from paper_conf_cgo_margiolaso16_b200.jobs import SgemmJob
    d = synth.preset("sgemm", "default")
    job = SgemmJob(d)
    acc.run([job])
    c = job.result()["c"]
    r = np.random.Generator(np.random.PCG64(2))
    ij = np.stack([r.integers(0, d["m"], 4000), r.integers(0, d["n"], 4000)], 1)
    ij = np.concatenate([ij, [[0, 0], [d["m"] - 1, d["n"] - 1], [127, 128], [128, 127]]])
    assert_close_fp32(c[ij[:, 0], ij[:, 1]], oracle_lib.sgemm_entries(d, ij), what="sgemm default")


def test_sgemm_identity():
    """B = I reproduces A (within fp32 rounding of a single product)."""
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no GPU")
    from paper_conf_cgo_margiolaso16_b200.jobs import SgemmJob
    from paper_conf_cgo_margiolaso16_b200.runtime import Accel
    k = 256
    a = synth.preset("sgemm", "tiny", k=k)["a"]
    d = {"a": a, "b": np.eye(k, dtype=np.float32), "m": a.shape[0], "n": k, "k": k}
    with Accel(0) as acc:
        job = SgemmJob(d)
        acc.run([job])
        assert np.array_equal(job.result()["c"], a)


@pytest.mark.parametrize("size,over", [("tiny", {}), ("small", dict(numk=1000)), ("tiny", dict(nvox_1d=7, numk=257))])
def test_mriq(acc_tiny_caps, oracle_lib, size, over):
    from paper_conf_cgo_margiolaso16_b200.jobs import MriqJob
    d = synth.preset("mriq", size, **over)
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: MriqJob(d))
    same(nat, sh)
    pm, qr, qi = oracle_lib.mriq(d)
    assert np.array_equal(sh["phimag"], pm)
    assert_close_fp32(np.concatenate([sh["qr"], sh["qi"]]), np.concatenate([qr, qi]), what="mri-q")


def test_mriq_default_sampled(acc, oracle_lib):
    from paper_conf_cgo_margiolaso16_b200.jobs import MriqJob
    d = synth.preset("mriq", "default")
    job = MriqJob(d)
    acc.run([job])
    res = job.result()
    pm = oracle_lib.mriq_phimag(d)
    assert np.array_equal(res["phimag"], pm)
    r = np.random.Generator(np.random.PCG64(5))
    idx = np.concatenate([r.integers(0, d["numx"], 1500), [0, d["numx"] - 1]])
    qr, qi = oracle_lib.mriq_points(d, idx, pm)
    assert_close_fp32(np.concatenate([res["qr"][idx], res["qi"][idx]]), np.concatenate([qr, qi]),
                      what="mri-q default")


# ---------------------------------------------------------------- sad (f3)
@pytest.mark.parametrize("size,over", [("tiny", {}), ("small", {}), ("tiny", dict(R=0)), ("tiny", dict(R=7, w=64))])
def test_sad(acc_tiny_caps, oracle_lib, size, over):
    """Parboil sad, three steps (4x4 SADs, 8x8 and 16x16 sums): bit-exact in
    both modes, every displacement parity and the frame-edge clamping."""
    from paper_conf_cgo_margiolaso16_b200.jobs import SadJob
    d = synth.preset("sad", size, **over)
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: SadJob(d))
    s4, s8, s16 = oracle_lib.sad(d)
    for r in (nat, sh):
        assert np.array_equal(r["sad4"], s4) and np.array_equal(r["sad8"], s8) and np.array_equal(r["sad16"], s16)


def test_sad_default(acc, oracle_lib):
    from paper_conf_cgo_margiolaso16_b200.jobs import SadJob
    d = synth.preset("sad", "default")
    nat, sh, _ = run_modes(acc, lambda: SadJob(d))
    s4, s8, s16 = oracle_lib.sad(d)
    for r in (nat, sh):
        assert np.array_equal(r["sad16"], s16) and np.array_equal(r["sad8"], s8) and np.array_equal(r["sad4"], s4)


# ---------------------------------------------------------------- lbm (f3)
@pytest.mark.parametrize("size,over", [("tiny", {}), ("small", {}), ("tiny", dict(nx=130, ny=5, nz=4, steps=4))])
def test_lbm(acc_tiny_caps, oracle_lib, size, over):
    """Parboil lbm (D3Q19 stream + BGK collide, bounce-back obstacles,
    periodic): NATIVE == SHARED bit-exact, both within 1e-4 of the fp64 oracle."""
    from paper_conf_cgo_margiolaso16_b200.jobs import LbmJob
    d = synth.preset("lbm", size, **over)
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: LbmJob(d))
    same(nat, sh)
    assert_close_fp32(sh["f"], oracle_lib.lbm(d), what="lbm")


def test_lbm_default(acc, oracle_lib):
    from paper_conf_cgo_margiolaso16_b200.jobs import LbmJob
    d = synth.preset("lbm", "default", steps=6)
    nat, sh, _ = run_modes(acc, lambda: LbmJob(d))
    same(nat, sh)
    assert_close_fp32(sh["f"], oracle_lib.lbm(d), what="lbm default")


# ---------------------------------------------------------------- mri-gridding (f3)
@pytest.mark.parametrize("size,over", [("tiny", {}), ("small", {}), ("tiny", dict(G=21, n=5000))])
def test_gridding(acc_tiny_caps, oracle_lib, size, over):
    """Parboil mri-gridding pipeline (binning, 3-kernel scan, reorder,
    gridding): NATIVE == SHARED bit-exact (fixed-point sums: independent of
    the atomic binning order), within 1e-4 of the fp64 oracle."""
    from paper_conf_cgo_margiolaso16_b200.jobs import GriddingJob
    d = synth.preset("gridding", size, **over)
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: GriddingJob(d))
    same(nat, sh)
    assert_close_fp32(sh["grid"], oracle_lib.gridding(d), what="gridding")


def test_gridding_default(acc, oracle_lib):
    from paper_conf_cgo_margiolaso16_b200.jobs import GriddingJob
    d = synth.preset("gridding", "default")
    nat, sh, _ = run_modes(acc, lambda: GriddingJob(d))
    same(nat, sh)
    assert_close_fp32(sh["grid"], oracle_lib.gridding(d), what="gridding default")


def test_mriq_slices_next_to_cutcp(acc, oracle_lib):
    """R-disp-9: in SHARED mode mri-q's Q launch runs as 4 VG ranges (1 + 4
    descriptors; NATIVE keeps 1 + 1), every VG exactly once (the fixture
    verifies coverage), results as the oracle, under both policies and with
    a cutcp request submitted while it runs (the co-runner it used to
    starve)."""
    import time
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import MriqJob, make_job
    d = synth.preset("mriq", "small")
    pm, qr, qi = oracle_lib.mriq(d)
    cut = make_job("cutcp", synth.preset("cutcp", "small"))
    try:
        for mode, pol, want in [(abi.MODE_NATIVE, abi.POLICY_STATIC, 2), (abi.MODE_SHARED, abi.POLICY_STATIC, 5),
                                (abi.MODE_SHARED, abi.POLICY_RESOLVE, 5)]:
            acc.set_mode(mode, pol)
            job = MriqJob(d)
            ids = acc.submit([job], tenants=[0])
            time.sleep(2e-4)
            ids += acc.submit([cut], tenants=[1])
            acc.sync()
            st = [acc.stats(i) for i in ids]
            acc.release()
            assert st[0].launches == want, (mode, pol, st[0].launches)
            assert st[0].coverage_ok == 1 and st[1].coverage_ok == 1
            res = job.result()
            assert np.array_equal(res["phimag"], pm)
            assert_close_fp32(np.concatenate([res["qr"], res["qi"]]), np.concatenate([qr, qi]), what="mri-q sliced")
    finally:
        acc.set_mode(abi.MODE_SHARED, abi.POLICY_STATIC)
