"""Small SHARED/NATIVE runs for compute-sanitizer (memcheck, racecheck,
synccheck): the dispatch protocol (Fig. 8b master dequeue + barrier, RESOLVE
admission/eviction) around tenants that stage with cp.async, TMA + mbarriers
and shared-memory atomics, next to bfs (the co-runner of the round-1 stale
TMA tile).  Tiny sizes: the sanitizers slow kernels down 10-100x.

    compute-sanitizer --tool racecheck python scripts/sanitize.py
"""
import os
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import numpy as np  # noqa: E402

import synth  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import StencilJob, make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402


def main():
    caps = abi.accel_caps(4, 2048, 65536, 233472, 32)   # 4 SMs' worth of quota: many VGs per CTA
    d = {"mop": synth.preset("mop", "tiny"), "bfs": synth.preset("bfs", "tiny"),
         "stencil": synth.preset("stencil", "tiny", nx=136, ny=17, nz=19, sweeps=3),
         "histo": synth.preset("histo", "tiny", bins=16384, sample_bytes=4),
         "tpacf": synth.preset("tpacf", "tiny"), "sgemm": synth.preset("sgemm", "tiny")}
    with Accel(device=0, mode=abi.MODE_SHARED, verify=True, caps=caps) as acc:
        for mode, pol in [(abi.MODE_NATIVE, abi.POLICY_STATIC), (abi.MODE_SHARED, abi.POLICY_STATIC),
                          (abi.MODE_SHARED, abi.POLICY_RESOLVE)]:
            acc.set_mode(mode, pol)
            outs = {}
            for kern in ("stencil_tma", "stencil"):
                jobs = [StencilJob(d["stencil"], kernel=kern), make_job("bfs", d["bfs"]), make_job("mop", d["mop"]),
                        make_job("histo", d["histo"]), make_job("tpacf", d["tpacf"]), make_job("sgemm", d["sgemm"])]
                st = acc.run(jobs)
                assert all(s.coverage_ok == 1 for s in st)
                outs[kern] = jobs[0].result()["a"]
            assert np.array_equal(outs["stencil_tma"], outs["stencil"])
            print("mode", mode, "policy", pol, "ok", flush=True)
    print("sanitize run ok")


if __name__ == "__main__":
    main()
