"""Per-tenant isolated timing: NATIVE vs SHARED (persistent, K=1) at a preset
size, per-launch CUDA-event times, achieved bandwidth / throughput.

    python scripts/isolated.py [--size default] [--reps 5] tenant ...
"""
import argparse
import json
import os
import statistics
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

import synth  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("tenants", nargs="+")
    ap.add_argument("--size", default="default")
    ap.add_argument("--reps", type=int, default=5)
    ap.add_argument("--chunk", type=int, default=0, help="override VGs per dequeue for all kernels")
    ap.add_argument("--policy", default="both", choices=["static", "resolve", "both"])
    args = ap.parse_args()
    from paper_conf_cgo_margiolaso16_b200 import abi as _abi
    chunks = {n: args.chunk for n in _abi.accel_builtin_names()} if args.chunk else None
    acc = Accel(0, chunks=chunks)
    flush = torch.empty(64 * 1024 * 1024, dtype=torch.float32, device="cuda")
    out = {}
    for t in args.tenants:
        d = synth.preset(t, args.size, seed=1)
        job = make_job(t, d)
        if hasattr(job, "fit_levels"):
            job.fit_levels(acc)
        res = {}
        pols = {"static": [abi.POLICY_STATIC], "resolve": [abi.POLICY_RESOLVE],
                "both": [abi.POLICY_STATIC, abi.POLICY_RESOLVE]}[args.policy]
        pname = {abi.POLICY_STATIC: "persistent", abi.POLICY_RESOLVE: "persistent_resolve"}
        runs = [(abi.MODE_NATIVE, "native", abi.POLICY_STATIC)] + [(abi.MODE_SHARED, pname[p], p) for p in pols]
        for mode, name, pol in runs:
            acc.set_mode(mode, pol)
            el, lt, q = [], [], 0
            for _ in range(args.reps + 1):
                flush.fill_(1)
                torch.cuda.synchronize()
                ids = acc.submit([job], launch_events=True)
                acc.sync()
                s = acc.stats(ids[0])
                el.append(s.elapsed_ms)
                lt.append(acc.launch_times(ids[0], job.launches()))
                q = s.quota_initial
                acc.release()
            el, lt = el[1:], lt[1:]
            w = job.work()
            # per-launch times of the MAIN step only (the GEMM, not its operand
            # split; mri-q's Q, not PhiMag): the roofline is that kernel's
            first = sum(st.repeat for st in job.steps[:job.main_step]) if job.main_step >= 0 else 0
            nmain = job.steps[job.main_step].repeat if job.main_step >= 0 else job.launches()
            per = [x for l in lt for x in l[first:first + nmain]]
            by_step, k = [], 0
            for st in job.steps:
                by_step.append(statistics.mean(x for l in lt for x in l[k:k + st.repeat]))
                k += st.repeat
            r = {"elapsed_ms": statistics.median(el), "launch_ms_mean": statistics.mean(per),
                 "launch_ms_min": min(per), "launch_ms_by_step": by_step, "quota": q}
            if w.get("bound") == "hbm":
                b = w.get("bytes_per_launch", w.get("bytes"))
                r["GBps_mean"] = b / r["launch_ms_mean"] / 1e6
            elif "flops" in w or "flops_per_launch" in w:
                f = w.get("flops_per_launch", w.get("flops"))
                r["TFLOPs_mean"] = f / r["launch_ms_mean"] / 1e9
            res[name] = r
        for nm in ("persistent", "persistent_resolve"):
            if nm in res:
                res["overhead" + nm[len("persistent"):]] = res[nm]["elapsed_ms"] / res["native"]["elapsed_ms"] - 1
        if "persistent_resolve" in res:
            res["overhead_resolve"] = res["persistent_resolve"]["elapsed_ms"] / res["native"]["elapsed_ms"] - 1
        info = acc.kernel_info(job.steps[0].kernel)
        res["regs"] = info.num_regs
        res["occ"] = [info.occ_native, info.occ_persistent]
        out[t] = res
        print(t, json.dumps(res), flush=True)
    acc.close()


if __name__ == "__main__":
    main()
