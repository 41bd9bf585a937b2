"""Where does the wrong zm plane staged by stencil_tma come from?  Run the TMA
stencil next to bfs with the dbg block, and look every recorded staged value
up in the reference volumes (the cp.async kernel after t sweeps): which
sweep and which z plane at the same (y, x) holds exactly that value.
    ACCEL_LIB=<build with -DACCEL_XP_TMA_DBG=1> python scripts/diag_tma_which.py [--sweeps 8] [--mode static]"""
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

ap = argparse.ArgumentParser()
ap.add_argument("--sweeps", type=int, default=8)
ap.add_argument("--mode", default="static")
ap.add_argument("--reps", type=int, default=4)
a = ap.parse_args()
_, _, inp = bench.make_inputs("c2", 0)
acc = Accel(0)
acc.set_mode(abi.MODE_NATIVE, abi.POLICY_STATIC)
ref = {0: inp["stencil"]["a0"]}
for t in range(1, a.sweeps + 1):
    j = StencilJob(dict(inp["stencil"], sweeps=t), kernel="stencil")
    acc.run([j])
    ref[t] = j.result()["a"]
bfs = make_job("bfs", inp["bfs"])
bfs.fit_levels(acc)
m = {"native": (abi.MODE_NATIVE, abi.POLICY_STATIC), "static": (abi.MODE_SHARED, abi.POLICY_STATIC),
     "resolve": (abi.MODE_SHARED, abi.POLICY_RESOLVE)}[a.mode]
acc.set_mode(*m)
dbg = torch.zeros(8 + 8 * 16, dtype=torch.int32, device="cuda")
for rep in range(a.reps):
    dbg.zero_()
    sj = StencilJob(dict(inp["stencil"], sweeps=a.sweeps), kernel="stencil_tma")
    sj.args.dbg = dbg.data_ptr()
    acc.run([bfs, sj])
    d = dbg.cpu().numpy().view(np.uint32)
    print(f"rep {rep}: {int(d[0])} mismatches", flush=True)
    for k in range(min(int(d[0]), 16)):
        rec = d[8 + 8 * k: 16 + 8 * k]
        r, z, y, x = int(rec[0]), int(rec[1]) & 0x3fffffff, int(rec[2]), int(rec[3])
        sv = np.float32(struct.unpack("f", struct.pack("I", int(rec[4])))[0])
        hits = [(t, zz) for t in ref for zz in range(ref[t].shape[0]) if ref[t][zz, y, x] == sv]
        print(f"    launch {r} plane z {z} (y {y}, x {x}): staged {sv:.9g} want {ref[r][z, y, x]:.9g}; "
              f"equal to (sweeps, z): {hits[:6]}", flush=True)
