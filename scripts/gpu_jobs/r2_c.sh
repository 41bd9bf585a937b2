#!/bin/bash
# round 2 batch c: stencil_tma parity + speed, GPU suite, bench, sanitizers
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 1200 python -m pytest tests -m gpu -x -q --timeout 600 -p no:cacheprovider > gpurun_out/r2c_gputest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r2c_gputest.log
tail -15 gpurun_out/r2c_gputest.log
python - <<'PY' > gpurun_out/r2c_stencil_iso.log 2>&1
import os, sys, statistics, torch
sys.path.insert(0, os.getcwd())
import synth
from paper_conf_cgo_margiolaso16_b200 import abi
from paper_conf_cgo_margiolaso16_b200.jobs import StencilJob
from paper_conf_cgo_margiolaso16_b200.runtime import Accel
d = synth.preset("stencil", "default", seed=1)
acc = Accel(0)
flush = torch.empty(64 << 20, dtype=torch.float32, device="cuda")
for kern in ("stencil_tma", "stencil"):
    job = StencilJob(d, kernel=kern)
    for mode, pol, nm in [(abi.MODE_NATIVE, abi.POLICY_STATIC, "native"), (abi.MODE_SHARED, abi.POLICY_STATIC, "static"), (abi.MODE_SHARED, abi.POLICY_RESOLVE, "resolve")]:
        acc.set_mode(mode, pol)
        ts = []
        for _ in range(8):
            flush.fill_(1); torch.cuda.synchronize()
            ids = acc.submit([job], launch_events=True); acc.sync()
            lt = acc.launch_times(ids[0], job.launches()); s = acc.stats(ids[0]); acc.release()
            ts.append((s.elapsed_ms, statistics.mean(lt), s.quota_initial))
        ts = ts[1:]
        el = statistics.median(t[0] for t in ts); per = statistics.median(t[1] for t in ts)
        print(kern, nm, "elapsed_ms %.4f per_launch_us %.2f GBps %.0f quota %d" % (el, per * 1e3, 8 * 512 * 512 * 64 / per / 1e6, ts[-1][2]), flush=True)
PY
cat gpurun_out/r2c_stencil_iso.log
timeout 300 python bench.py --steps 10 --warmup 3 > gpurun_out/r2c_bench.log 2>&1
tail -c 700 gpurun_out/r2c_bench.log
for tool in memcheck racecheck synccheck; do
  timeout 900 compute-sanitizer --tool $tool --print-limit 20 python scripts/sanitize.py > gpurun_out/r2c_san_$tool.log 2>&1
  echo "$tool rc=$?"; tail -4 gpurun_out/r2c_san_$tool.log
done
