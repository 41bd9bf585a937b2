#!/bin/bash
# stencil staging variants vs device share (alone) and in the C2 bench
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
for k in stencil stencil_deep stencil_tma; do
  echo "== $k"
  ACCEL_STENCIL_KERNEL=$k timeout 300 python scripts/share_profile.py --tenants stencil --fracs 1,0.5,0.25,0.125 --reps 3 2>&1 | grep "^stencil"
done
for k in stencil stencil_deep; do
  ACCEL_STENCIL_KERNEL=$k timeout 600 python bench.py --no-cpu-baseline --out gpurun_out/ss_bench_$k.json > gpurun_out/ss_bench_$k.log 2>&1
  python -c "
import json; d=json.load(open('gpurun_out/ss_bench_$k.json')); s=d['sharing']
print('$k', round(d['value'],1), 'native', round(s['native_mixes_per_s'],1), 'U', round(s['unfairness_shared'],3), 'STP', round(s['stp_ratio'],3), {k: round(v,2) for k,v in s['T_s_ms_shared'].items()}, 'frac', round(d['roofline']['frac'],3), s['quotas_last_step']['stencil'])"
done
