"""Per-VG execution trace of one tenant, native vs persistent (STATIC):
VG duration, per-CTA dequeue gaps, per-SM finish spread (tail), SM idle.
    python scripts/vg_trace.py tenant [size] [--launch L]"""
import argparse
import os
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import synth  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402


def analyse(tr, label):
    ran = tr[tr["t_start_ns"] > 0]
    t0 = ran["t_start_ns"].min()
    s = (ran["t_start_ns"] - t0) / 1e3
    e = (ran["t_end_ns"] - t0) / 1e3
    dur = e - s
    span = e.max()
    out = {"label": label, "vgs": int(len(ran)), "span_us": round(float(span), 1),
           "vg_us_mean": round(float(dur.mean()), 2), "vg_us_p50": round(float(np.median(dur)), 2),
           "vg_us_max": round(float(dur.max()), 2)}
    sms = ran["sm"]
    busy = np.zeros(sms.max() + 1)
    last = np.zeros(sms.max() + 1)
    np.add.at(busy, sms, dur)
    np.maximum.at(last, sms, e)
    out["sm_last_end_us_min/med"] = (round(float(last.min()), 1), round(float(np.median(last)), 1))
    # running VGs over time: fraction of span with fewer than 90 % of peak concurrency
    ev = np.concatenate([np.stack([s, np.ones_like(s)], 1), np.stack([e, -np.ones_like(e)], 1)])
    ev = ev[np.argsort(ev[:, 0], kind="stable")]
    run = np.cumsum(ev[:, 1])
    peak = run.max()
    dt = np.diff(ev[:, 0], append=ev[-1, 0])
    out["peak_running"] = int(peak)
    out["avg_running"] = round(float((run * dt).sum() / span), 1)
    out["frac_below_90pct"] = round(float(dt[run < 0.9 * peak].sum() / span), 3)
    cnt = np.bincount(sms)
    out["vgs_per_sm_min/max"] = (int(cnt[cnt > 0].min()), int(cnt.max()))
    out["sm_busy_us_min/max"] = (round(float(busy[cnt > 0].min()), 0), round(float(busy.max()), 0))
    slow = np.argsort(dur)[-5:]
    vid = np.nonzero(tr["t_start_ns"] > 0)[0]
    out["slowest(vg,sm,start,dur)"] = [(int(vid[i]), int(sms[i]), round(float(s[i]), 0), round(float(dur[i]), 0)) for i in slow]
    # per-CTA gaps between consecutive VGs (persistent only)
    cta = ran["cta"]
    if len(np.unique(cta)) < len(ran):
        o = np.lexsort((s, cta))
        cs, ss, es = cta[o], s[o], e[o]
        same = cs[1:] == cs[:-1]
        gaps = ss[1:][same] - es[:-1][same]
        out["gap_us_mean/p50/max"] = (round(float(gaps.mean()), 2), round(float(np.median(gaps)), 2),
                                      round(float(gaps.max()), 2))
        first = np.array([ss[cs == c].min() for c in np.unique(cs)])
        per_cta = np.bincount(np.unique(cs, return_inverse=True)[1])
        out["vgs_per_cta_hist"] = np.bincount(per_cta).tolist()
        # within each SM: VG count of its CTAs (slot -> priority effect)
        sm_of = {}
        for c_, m_ in zip(cta, sms):
            sm_of[int(c_)] = int(m_)
        out["cta_first_start_us_max"] = round(float(first.max()), 2)
    return out


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("tenant")
    ap.add_argument("size", nargs="?", default="default")
    ap.add_argument("--launch", type=int, default=-1, help="launch index to analyse (-1: the longest)")
    ap.add_argument("--policy", default="static", choices=["static", "resolve"])
    a = ap.parse_args()
    d = synth.preset(a.tenant, a.size, seed=1)
    for mode in ("native", "persistent"):
        acc = Accel(0, mode=abi.MODE_NATIVE if mode == "native" else abi.MODE_SHARED,
                    policy=abi.POLICY_RESOLVE if a.policy == "resolve" else abi.POLICY_STATIC)
        job = make_job(a.tenant, d)
        acc.run([job])                      # warm
        ids = acc.submit([job], trace=True)
        acc.sync()
        tr = acc.vg_trace(ids[0])
        ls = acc.launch_stats(ids[0], 4096)
        acc.release()
        acc.close()
        # split the trace per launch with the static totals of each launch
        totals = [job.steps[i].grid[0] * job.steps[i].grid[1] * job.steps[i].grid[2] for i in range(len(job.steps))
                  for _ in range(job.steps[i].repeat)]
        offs = np.concatenate([[0], np.cumsum(totals)])
        spans = [(tr[offs[i]:offs[i + 1]]["t_end_ns"].max() - tr[offs[i]:offs[i + 1]]["t_start_ns"][tr[offs[i]:offs[i + 1]]["t_start_ns"] > 0].min())
                 if (tr[offs[i]:offs[i + 1]]["t_start_ns"] > 0).any() else 0 for i in range(len(totals))]
        li = int(np.argmax(spans)) if a.launch < 0 else a.launch
        if len(ls) > 1:
            lsp = [(l.t_last_ns - l.t_first_ns) / 1e3 for l in ls]
            gaps = [(ls[i + 1].t_first_ns - ls[i].t_last_ns) / 1e3 for i in range(len(ls) - 1)]
            print(a.tenant, mode, "launches", len(ls), "span us mean %.1f" % np.mean(lsp),
                  "gap us mean %.2f min %.2f" % (np.mean(gaps), np.min(gaps)),
                  "request us %.1f" % ((ls[-1].t_last_ns - ls[0].t_first_ns) / 1e3), flush=True)
        part = tr[offs[li]:offs[li + 1]]
        print(a.tenant, mode, "launch", li, analyse(part, mode), flush=True)
        dur = (part["t_end_ns"].astype(np.int64) - part["t_start_ns"].astype(np.int64)) / 1e3
        nb = 16
        edges = np.linspace(0, len(part), nb + 1).astype(int)
        print("  mean VG us per id bucket:", [round(float(dur[edges[i]:edges[i + 1]].mean()), 0) for i in range(nb)])
        st0 = (part["t_start_ns"] - part["t_start_ns"][part["t_start_ns"] > 0].min()) / 1e3
        w1 = st0 < 5
        print("  first-wave VGs:", int(w1.sum()), "mean us", round(float(dur[w1].mean()), 0),
              "later mean us", round(float(dur[~w1].mean()), 0))
        fw = part[w1]
        fd = dur[w1]
        ratios = []
        for smv in np.unique(fw["sm"]):
            dd = fd[fw["sm"] == smv]
            if len(dd) > 1:
                ratios.append(dd.max() / max(dd.min(), 1e-3))
        print("  first wave, per SM max/min VG duration: median %.2f p90 %.2f" %
              (float(np.median(ratios)), float(np.percentile(ratios, 90))))
        del ls
        torch.cuda.synchronize()


if __name__ == "__main__":
    main()
