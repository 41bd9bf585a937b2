for v in dyn dyn2 stride; do echo "== $v"; ACCEL_DISPATCH=$v timeout 600 python scripts/isolated.py spmv histo stencil bfs tpacf cutcp --reps 3 2>&1 | python -c "
import sys,json
for l in sys.stdin:
  n,j=l.split(' ',1); j=json.loads(j); print(n, 'native %.1f us/launch' % (1e3*j['native']['launch_ms_mean']), 'persistent %.1f' % (1e3*j['persistent']['launch_ms_mean']), 'overhead %.3f' % j['overhead'])
"; done
