#!/bin/bash
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tenants.py tests/test_gpu_order.py -k "cutcp or tpacf or order" -q -x --timeout 300 -p no:cacheprovider 2>&1 | tail -3
timeout 300 python scripts/isolated.py --reps 8 cutcp tpacf 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    try:
        t,j=l.split(' ',1); r=json.loads(j)
    except Exception: continue
    print(t, 'native %.4f static %.4f resolve %.4f  ov_static %.4f ov_resolve %.4f' % (r['native']['elapsed_ms'], r['persistent']['elapsed_ms'], r['persistent_resolve']['elapsed_ms'], r['overhead'], r['overhead_resolve']))" | tee gpurun_out/r2v_iso.log
timeout 300 python bench.py --steps 10 --warmup 3 --no-cpu-baseline --out gpurun_out/r2v_bench.json > gpurun_out/r2v_bench.log 2>&1
python -c "
import json; b=json.load(open('gpurun_out/r2v_bench.json')); print(b['headline']); print({k:round(v,3) for k,v in b['sharing']['T_s_ms_shared'].items()}, {k:round(v,3) for k,v in b['sharing']['T_a_ms'].items()})"
