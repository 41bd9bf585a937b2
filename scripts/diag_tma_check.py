"""TMA stencil drift next to bfs: does the staged plane differ from an L2 load
of the same input at the moment the consumer reads it?  (stencil_tma's
diagnostic `dbg` block: every staged row of every plane is compared with
__ldcg of the input buffer; mismatches are counted and the first 16 recorded
with the output buffer's value at the same point.)
    ACCEL_LIB=<build with -DACCEL_XP_TMA_DBG=1> python scripts/diag_tma_check.py [--kernel stencil_tma] [--reps 3]"""
import argparse
import os
import struct
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import bench  # noqa: E402
from paper_conf_cgo_margiolaso16_b200 import abi  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.jobs import StencilJob, make_job  # noqa: E402
from paper_conf_cgo_margiolaso16_b200.runtime import Accel  # noqa: E402


def f(b):
    return struct.unpack("f", struct.pack("I", int(b)))[0]


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--kernel", default="stencil_tma")
    ap.add_argument("--reps", type=int, default=3)
    ap.add_argument("--sweeps", type=int, default=100)
    ap.add_argument("--l2hint", type=int, default=0, help="diagnostic bits (stencil_tma.cuh)")
    a = ap.parse_args()
    _, _, inp = bench.make_inputs("c2", 0)
    ds = dict(inp["stencil"], sweeps=a.sweeps)
    acc = Accel(0)
    acc.set_mode(abi.MODE_NATIVE, abi.POLICY_STATIC)
    ref = StencilJob(ds, kernel="stencil")
    acc.run([ref])
    want = ref.result()["a"]
    bfs = make_job("bfs", inp["bfs"])
    bfs.fit_levels(acc)
    dbg = torch.zeros(8 + 8 * 16, dtype=torch.int32, device="cuda")
    for pol_name, mode, pol in [("native", abi.MODE_NATIVE, abi.POLICY_STATIC),
                                ("static", abi.MODE_SHARED, abi.POLICY_STATIC),
                                ("resolve", abi.MODE_SHARED, abi.POLICY_RESOLVE)]:
        acc.set_mode(mode, pol)
        for co in (["bfs"],):
            for rep in range(a.reps):
                dbg.zero_()
                sj = StencilJob(ds, kernel=a.kernel)
                sj.args.dbg = dbg.data_ptr()
                sj.args.l2hint = a.l2hint
                acc.run(([bfs] if co else []) + [sj])
                got = sj.result()["a"]
                d = dbg.cpu().numpy().view(np.uint32)
                msg = (f"{pol_name:8s} co={'+'.join(co) or '-':4s} rep {rep}: output differs at "
                       f"{int((got != want).sum())} points; staged != L2 at {int(d[0])} points")
                tags = {}
                for k in range(min(int(d[0]), 16)):
                    rec = d[8 + 8 * k: 16 + 8 * k]
                    key = (int(rec[1]) >> 30, int(rec[7]) if (int(rec[1]) >> 30) == 3 else -1)
                    tags[key] = tags.get(key, 0) + 1
                print(msg + f"  first-16 by (tag, plane): {tags}", flush=True)
                for k in range(min(int(d[0]), 4)):
                    rec = d[8 + 8 * k: 16 + 8 * k]
                    print(f"    launch {rec[0]} z {rec[1] & 0x3fffffff} tag {rec[1] >> 30} y {rec[2]} x {rec[3]}: staged {f(rec[4]):.9g} "
                          f"L2 {f(rec[5]):.9g} output-buffer {f(rec[7]):.9g} sm {rec[6]}", flush=True)


if __name__ == "__main__":
    main()
