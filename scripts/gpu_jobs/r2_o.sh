#!/bin/bash
# attribute the RESOLVE per-launch overhead with the measurement-only ablations
# (ACCEL_ABLATE bits: 1 no retire fence, 2 no live-quota load, 4 no stats red,
#  8 no alive decrement, 16 no predecessor topped check) -- isolated, K = 1
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
for ab in 0 1 16 17 2 8 9 31; do
  echo "== ACCEL_ABLATE=$ab"
  ACCEL_ABLATE=$ab timeout 300 python scripts/isolated.py --reps 8 --policy resolve stencil spmv lbm 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    t,j=l.split(' ',1); r=json.loads(j)
    print(t, 'native %.4f resolve %.4f overhead %.4f' % (r['native']['elapsed_ms'], r['persistent_resolve']['elapsed_ms'], r['overhead_resolve']))"
done 2>&1 | tee gpurun_out/r2o_ablate.log
