#!/bin/bash
# stencil_z16 (16 planes per VG) vs stencil: parity, share profile, C2 bench
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_tenants.py -q -x -p no:cacheprovider -k "stencil" 2>&1 | tail -2
for k in stencil stencil_z16; do
  echo "== $k"
  ACCEL_STENCIL_KERNEL=$k timeout 300 python scripts/share_profile.py --tenants stencil --fracs 1,0.5,0.25,0.125 --reps 3 2>&1 | grep "^stencil"
  for rep in 1 2; do
    ACCEL_STENCIL_KERNEL=$k timeout 600 python bench.py --no-cpu-baseline --out gpurun_out/z16_bench_$k.json > /dev/null 2>&1
    python -c "
import json; d=json.load(open('gpurun_out/z16_bench_$k.json')); s=d['sharing']
print('$k bench', round(d['value'],1), 'native', round(s['native_mixes_per_s'],1), 'U', round(s['unfairness_shared'],3), 'STP', round(s['stp_ratio'],3), {k: round(v,2) for k,v in s['T_s_ms_shared'].items()}, 'frac', round(d['roofline']['frac'],3), 'iso', round(d['roofline']['isolated']['frac'],3), 'ovh', d['headline']['max_dispatch_overhead'])"
  done
done
