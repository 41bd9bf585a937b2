"""Diagnostic: staggered RESOLVE/STATIC mix vs an isolated NATIVE stencil run
(bit-exact expected: same kernel body, same per-cell arithmetic)."""
import os, sys, time
os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import synth
from paper_conf_cgo_margiolaso16_b200 import abi
from paper_conf_cgo_margiolaso16_b200.jobs import BfsJob, HistoJob, SgemmTcJob, StencilJob, TpacfJob
from paper_conf_cgo_margiolaso16_b200.runtime import Accel

seed = 0
SW = int(os.environ.get("SWEEPS", "30"))
dsn = synth.preset("stencil", "default", seed=seed, sweeps=SW)
VICTIM = os.environ.get("VICTIM", "stencil")
def victim(vs):
    if VICTIM == "stencil":
        return StencilJob(dsn)
    return SgemmTcJob(synth.preset("sgemm", os.environ.get("SGSIZE", "small"), seed=vs))
def vres(j):
    return j.result()["a"] if VICTIM == "stencil" else j.result()["c"]
nat = Accel(0, mode=abi.MODE_NATIVE)
refs = {}
for vs in range(3 if VICTIM != "stencil" else 1):
    jn = victim(vs)
    nat.run([jn])
    refs[vs] = vres(jn).copy()
nat.close()
for pol in sys.argv[1:] or ["resolve", "static"]:
    acc = Accel(0, mode=abi.MODE_NATIVE if pol == "native" else abi.MODE_SHARED,
                policy=abi.POLICY_RESOLVE if pol == "resolve" else abi.POLICY_STATIC, verify=os.environ.get("VERIFY", "1") == "1")
    for rep in range(3):
        mk = {"bfs": lambda: BfsJob(synth.preset("bfs", "default", seed=seed)),
              "histo": lambda: HistoJob(synth.preset("histo", "default", seed=seed, iters=8)),
              "tpacf": lambda: TpacfJob(synth.preset("tpacf", "small", seed=seed)),
              "stencil": lambda: StencilJob(dsn)}
        vs = rep if VICTIM != "stencil" else 0
        ref = refs[vs]
        jobs = [victim(vs)] + [mk[t]() for t in os.environ.get("MIXWITH", "bfs,histo,tpacf").split(",") if t]
        ids = []
        for t, j in enumerate(jobs):
            ids += acc.submit([j], tenants=[t])
            time.sleep(0.0002)
        acc.sync()
        st = [acc.stats(i) for i in ids]
        ls = acc.launch_stats(ids[0], SW if VICTIM == "stencil" else 3)
        acc.release()
        got = vres(jobs[0])
        bad = np.argwhere(got != ref)
        print(pol, rep, "cov", [s.coverage_ok for s in st], "resolves", [s.resolves for s in st], "bad", len(bad))
        if len(bad):
            zs = np.unique(bad[:, 0]); print("  z", zs[:20], "y", np.unique(bad[:, 1])[:20], "x", np.unique(bad[:, 2])[:20])
            print("  max abs", np.abs(got - ref).max())
            if len(bad) < 200: print("  cells", bad[:60].tolist())
            import scipy.ndimage as ndi
            err = np.abs(got.astype(np.float64) - ref)
            lab, nb = ndi.label(err > 0)
            print("  blobs", nb)
            for bi in range(1, min(nb, 8) + 1):
                m = lab == bi
                idx = np.argwhere(m)
                e = np.where(m, err, 0)
                am = np.unravel_index(e.argmax(), e.shape)
                print("   blob", bi, "cells", len(idx), "argmax", tuple(int(v) for v in am), "max", e.max(),
                      "bbox", idx.min(0).tolist(), idx.max(0).tolist())
        ov = [(i, (ls[i + 1].t_first_ns - ls[i].t_last_ns)) for i in range(len(ls) - 1) if ls[i + 1].t_first_ns < ls[i].t_last_ns]
        print("  overlaps (launch, ns):", ov[:20])
        t0 = ls[0].t_first_ns
        print("  spans us:", [((l.t_first_ns - t0) / 1e3, (l.t_last_ns - t0) / 1e3) for l in ls][:6])
    acc.close()
