timeout 1500 python -m pytest tests -m gpu -q -x 2>&1 | tail -3
timeout 600 python scripts/isolated.py stencil histo bfs cutcp tpacf spmv sgemm mriq --reps 3 2>&1 | python -c "
import sys,json
for l in sys.stdin:
  n,j=l.split(' ',1); j=json.loads(j); print(n, 'native %.1f us/launch' % (1e3*j['native']['launch_ms_mean']), 'persistent %.1f' % (1e3*j['persistent']['launch_ms_mean']), 'overhead %.3f' % j['overhead'], j['regs'])
"
