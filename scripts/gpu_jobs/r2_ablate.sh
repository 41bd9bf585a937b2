#!/bin/bash
# RESOLVE per-launch cost, one switch at a time (ACCEL_ABLATE bits, dispatch.cuh kAbl*)
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
for a in ${ABLATE_SET:-0 16 4 2 20 22}; do
  echo "== ACCEL_ABLATE=$a"
  ACCEL_ABLATE=$a timeout 300 python scripts/isolated.py --reps 8 --policy resolve ${ABL_TENANTS:-stencil lbm spmv cutcp} 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    if l[:1].isalpha() and '{' in l:
        n,j=l.split(' ',1); j=json.loads(j)
        print(f\"{n:10s} native {j['native']['launch_ms_mean']*1e3:8.2f} resolve {j['persistent_resolve']['launch_ms_mean']*1e3:8.2f} us/launch  elapsed overhead {j['overhead_resolve']*100:+.1f}%\")"
done
