"""GPU: the useful-occupancy cap (R-solver-9) bounds a kernel's quota alone
and leaves its results unchanged; co-runners get the rest."""
import numpy as np
import pytest

import synth
from tests.test_gpu_tenants import acc  # noqa: F401

pytestmark = pytest.mark.gpu


def test_mriq_alone_capped(acc, oracle_lib):
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import MriqJob
    acc.set_mode(abi.MODE_SHARED, abi.POLICY_STATIC)
    d = synth.preset("mriq", "small")
    job = MriqJob(d)
    s = acc.run([job])[0]
    import torch
    sms = torch.cuda.get_device_properties(0).multi_processor_count
    assert s.quota_initial <= 2 * sms
    nat = MriqJob(d)
    acc.set_mode(abi.MODE_NATIVE, abi.POLICY_STATIC)
    acc.run([nat])
    acc.set_mode(abi.MODE_SHARED, abi.POLICY_STATIC)
    for k in ("qr", "qi"):
        assert np.array_equal(job.result()[k], nat.result()[k])


def test_capped_tenant_leaves_room(acc):
    """mri-q (cap 2/SM) next to stencil: mri-q never exceeds its cap and the
    solver gives stencil at least the equal share."""
    import torch
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import MriqJob, StencilJob
    sms = torch.cuda.get_device_properties(0).multi_processor_count
    acc.set_mode(abi.MODE_SHARED, abi.POLICY_STATIC)
    m = MriqJob(synth.preset("mriq", "default"))
    st = StencilJob(synth.preset("stencil", "default", sweeps=2))
    sm, ss = acc.run([m, st])
    assert sm.quota_initial <= 2 * sms
    assert ss.quota_initial >= sm.quota_initial
