"""GPU: the useful-occupancy cap (R-solver-10) bounds a kernel's quota while
it shares the device, not alone, and leaves its results unchanged."""
import numpy as np
import pytest

import synth
from tests.test_gpu_tenants import acc  # noqa: F401

pytestmark = pytest.mark.gpu


def _sms():
    import torch
    return torch.cuda.get_device_properties(0).multi_processor_count


def test_mriq_alone_not_capped(acc):
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import MriqJob
    acc.set_mode(abi.MODE_SHARED, abi.POLICY_STATIC)
    d = synth.preset("mriq", "default")     # 8192 VGs: more than one CTA per SM alone
    job = MriqJob(d)
    s = acc.run([job])[0]
    assert s.quota_initial > _sms()          # alone: the full share
    nat = MriqJob(d)
    acc.set_mode(abi.MODE_NATIVE, abi.POLICY_STATIC)
    acc.run([nat])
    acc.set_mode(abi.MODE_SHARED, abi.POLICY_STATIC)
    for k in ("qr", "qi"):
        assert np.array_equal(job.result()[k], nat.result()[k])


@pytest.mark.parametrize("policy", ["static", "resolve"])
def test_capped_in_mix(acc, policy):
    """mri-q (cap 1 CTA/SM) next to stencil: mri-q holds at most one CTA per
    SM, stencil gets the rest, both results exact."""
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import MriqJob, StencilJob
    acc.set_mode(abi.MODE_SHARED, abi.POLICY_STATIC if policy == "static" else abi.POLICY_RESOLVE)
    dm = synth.preset("mriq", "default")
    m = MriqJob(dm)
    st = StencilJob(synth.preset("stencil", "default", sweeps=4))
    sm, ss = acc.run([m, st])
    assert sm.quota_initial <= _sms()
    assert ss.quota_initial > sm.quota_initial
    acc.set_mode(abi.MODE_NATIVE, abi.POLICY_STATIC)
    ref = MriqJob(dm)
    acc.run([ref])
    acc.set_mode(abi.MODE_SHARED)
    for k in ("qr", "qi"):
        assert np.array_equal(m.result()[k], ref.result()[k])
