#!/bin/bash
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tenants.py tests/test_gpu_resolve.py -k "stencil or resolve or grow or stagger" -q -x --timeout 300 -p no:cacheprovider 2>&1 | tail -3
timeout 300 python scripts/stencil_iso.py stencil stencil_deep 2>&1 | tee gpurun_out/r2p_stencil_iso.log
for c in 1 2 4; do
  echo "== chunk $c"
  timeout 400 python scripts/isolated.py --reps 8 --chunk $c spmv lbm stencil histo bfs 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    try:
        t,j=l.split(' ',1); r=json.loads(j)
    except Exception: continue
    print(t, 'native %.4f static %.4f resolve %.4f  ov_static %.4f ov_resolve %.4f' % (r['native']['elapsed_ms'], r['persistent']['elapsed_ms'], r['persistent_resolve']['elapsed_ms'], r['overhead'], r['overhead_resolve']))"
done 2>&1 | tee gpurun_out/r2p_chunks.log
