"""GPU: sgemm on tcgen05 tensor cores (3xTF32) vs the fp64 oracle, both modes."""
import numpy as np
import pytest

import synth
from tests.gpu_util import assert_close_fp32
from tests.test_gpu_tenants import acc, acc_tiny_caps, run_modes, same  # noqa: F401

pytestmark = pytest.mark.gpu


@pytest.mark.parametrize("size,over", [("tiny", dict(m=256, n=512, k=64)), ("tiny", {}),
                                       ("small", {}), ("tiny", dict(m=129, n=257, k=36)),
                                       ("tiny", dict(m=130, n=140, k=70)),     # k % 4 == 2: padded hi/lo rows
                                       ("tiny", dict(m=64, n=33, k=33)),       # k % 4 == 1, k not a slab multiple
                                       ("tiny", dict(m=5, n=7, k=3)),
                                       ("tiny", dict(m=300, n=600, k=100)),    # k % 32 == 4: one-step ragged slab
                                       ("tiny", dict(m=7, n=9, k=4))])
@pytest.mark.parametrize("one_step", [True, False], ids=["onestep", "twostep"])
def test_sgemm_tc(acc_tiny_caps, oracle_lib, size, over, one_step):
    from paper_conf_cgo_margiolaso16_b200.jobs import SgemmTcJob
    d = synth.preset("sgemm", size, **over)
    made = []
    nat, sh, _ = run_modes(acc_tiny_caps, lambda: made.append(SgemmTcJob(d, one_step=one_step)) or made[-1])
    assert made[-1].one_step == (one_step and d["k"] % 4 == 0)
    same(nat, sh)
    assert_close_fp32(sh["c"], oracle_lib.sgemm(d), what="sgemm_tc")


@pytest.mark.parametrize("one_step", [True, False], ids=["onestep", "twostep"])
def test_sgemm_tc_default_sampled(acc, oracle_lib, one_step):
    from paper_conf_cgo_margiolaso16_b200.jobs import SgemmTcJob
    d = synth.preset("sgemm", "default")
    job = SgemmTcJob(d, one_step=one_step)
    assert job.one_step == one_step and len(job.steps) == (1 if one_step else 2)
    acc.run([job])
    c = job.result()["c"]
    r = np.random.Generator(np.random.PCG64(3))
    ij = np.stack([r.integers(0, d["m"], 4000), r.integers(0, d["n"], 4000)], 1)
    ij = np.concatenate([ij, [[0, 0], [d["m"] - 1, d["n"] - 1], [127, 255], [128, 256]]])
    assert_close_fp32(c[ij[:, 0], ij[:, 1]], oracle_lib.sgemm_entries(d, ij), what="sgemm_tc default")


def test_one_tf32_product_would_fail_the_bound(oracle_lib):
    """Sanity of the tolerance: a single TF32 product (A_hi.B_hi)
    misses 1e-4, so the 3xTF32 correction terms are necessary."""
    d = synth.preset("sgemm", "tiny", k=512)
    def tf32(x):
        u = x.view(np.uint32).astype(np.uint64)
        u = ((u + 0x1000) & ~np.uint64(0x1FFF)).astype(np.uint32)
        return u.view(np.float32)
    one = tf32(d["a"]).astype(np.float64) @ tf32(d["b"]).astype(np.float64).T
    ref = oracle_lib.sgemm(d)
    with pytest.raises(AssertionError):
        assert_close_fp32(one, ref)
