#!/bin/bash
# A/B of library builds (ACCEL_LIB) on the stencil share profile, isolated overheads and the C2 bench.
# usage: LIBS="default ab/libaccel_x.so ..." bash scripts/gpu_jobs/r2_libab.sh
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
for L in ${LIBS:-default}; do
  if [ "$L" = default ]; then unset ACCEL_LIB; else export ACCEL_LIB=$PWD/$L; fi
  tag=$(basename $L .so)
  echo "======== $tag"
  [ -n "$AB_SHARE" ] && timeout 300 python scripts/share_profile.py --tenants ${AB_SHARE} --fracs 1,0.25 --reps 3 2>&1 | grep -v "^{"
  [ -n "$AB_ISO" ] && timeout 300 python scripts/isolated.py --reps 8 $AB_ISO 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    if l[:1].isalpha() and '{' in l:
        n,j=l.split(' ',1); j=json.loads(j)
        print(f\"{n:10s} static {j['overhead']*100:+.1f}% resolve {j['overhead_resolve']*100:+.1f}% launch us nat {j['native']['launch_ms_mean']*1e3:.1f} st {j['persistent']['launch_ms_mean']*1e3:.1f} rs {j['persistent_resolve']['launch_ms_mean']*1e3:.1f}\")"
  for rep in ${AB_BENCH_REPS:-1}; do
    timeout 600 python bench.py --no-cpu-baseline --out gpurun_out/ab_$tag.json > gpurun_out/ab_$tag.log 2>&1
    python -c "
import json; d=json.load(open('gpurun_out/ab_$tag.json')); s=d['sharing']
print('bench', round(d['value'],1), 'native', round(s['native_mixes_per_s'],1), 'U', round(s['unfairness_shared'],3), 'STP', round(s['stp_ratio'],3), {k: round(v,2) for k,v in s['T_s_ms_shared'].items()}, 'frac', round(d['roofline']['frac'],3), 'ovh', d['headline']['max_dispatch_overhead'])"
  done
done
