"""GPU: the per-VG trace (ACCEL_REQ_TRACE) records every virtual group of a
request exactly once, on a real SM, inside the launch's time window, and --
for the persistent kernel -- only on the CTAs of the quota."""
import numpy as np
import pytest

import synth

pytestmark = pytest.mark.gpu


@pytest.mark.parametrize("mode", ["native", "persistent"])
def test_trace_covers_every_vg(mode):
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no GPU")
    from paper_conf_cgo_margiolaso16_b200 import abi
    from paper_conf_cgo_margiolaso16_b200.jobs import HistoJob
    from paper_conf_cgo_margiolaso16_b200.runtime import Accel
    acc = Accel(0, mode=abi.MODE_NATIVE if mode == "native" else abi.MODE_SHARED)
    d = synth.preset("histo", "small", seed=4, iters=3)
    job = HistoJob(d)
    ids = acc.submit([job], trace=True)
    acc.sync()
    tr = acc.vg_trace(ids[0])
    st = acc.stats(ids[0])
    ls = acc.launch_stats(ids[0], 16)
    acc.release()
    acc.close()
    assert len(tr) == st.vgs_total
    assert (tr["t_start_ns"] > 0).all()
    assert (tr["t_end_ns"] >= tr["t_start_ns"]).all()
    n_sm = torch.cuda.get_device_properties(0).multi_processor_count
    assert (tr["sm"] < n_sm).all()
    per = st.vgs_total // st.launches
    for i, l in enumerate(ls):
        part = tr[i * per:(i + 1) * per]
        assert part["t_start_ns"].min() >= l.t_first_ns and part["t_end_ns"].max() <= l.t_last_ns
        if mode == "persistent":
            assert len(np.unique(part["cta"])) <= st.quota_max
