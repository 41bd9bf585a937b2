#!/bin/bash
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 600 python scripts/histo_iso.py 16384 32768 61440 2>&1 | tee gpurun_out/r2h_histo.log
timeout 300 python scripts/stencil_iso.py stencil stencil_deep 2>&1 | tee gpurun_out/r2h_stencil_iso.log
for k in stencil stencil_deep; do
  ACCEL_STENCIL_KERNEL=$k timeout 300 python bench.py --steps 8 --warmup 3 --no-cpu-baseline > gpurun_out/r2h_bench_$k.log 2>&1
  echo "== $k"; python -c "
import json,sys
l=[x for x in open('gpurun_out/r2h_bench_$k.log') if x.startswith('{')][0]; b=json.loads(l); s=b['sharing']
print(b['headline']); print({k:round(v,3) for k,v in s['T_s_ms_shared'].items()}, round(b['roofline']['frac'],3))"
done
timeout 1500 python -m pytest tests -m gpu -q --timeout 600 -p no:cacheprovider > gpurun_out/r2h_gputest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r2h_gputest.log; tail -8 gpurun_out/r2h_gputest.log
