timeout 1500 python -m pytest tests -m gpu -q -x 2>&1 | tail -4
timeout 600 python scripts/isolated.py stencil histo bfs cutcp tpacf spmv sgemm mriq --reps 3 2>&1 | python -c "
import sys,json
for l in sys.stdin:
  n,j=l.split(' ',1); j=json.loads(j); print(n, 'native %.1f us/launch' % (1e3*j['native']['launch_ms_mean']), 'persistent %.1f' % (1e3*j['persistent']['launch_ms_mean']), 'overhead %.3f' % j['overhead'], {k:round(v,1) for k,v in j['native'].items() if 'GB' in k or 'TF' in k})
"
timeout 900 python bench.py --steps 5 --warmup 3 --out gpurun_out/bench_c2_r4.json 2>&1 | tail -1 | python -c "
import sys,json; j=json.loads(sys.stdin.read()); print(json.dumps({k:j[k] for k in ('value','ms_per_step','e2e')})); print(json.dumps(j['sharing'])); print(json.dumps(j['roofline']))"
