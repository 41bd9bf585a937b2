timeout 1200 python -m pytest tests -m gpu -q -x 2>&1 | tail -2
for i in 1 2; do timeout 300 python -m pytest tests/test_gpu_resolve.py -q -x 2>&1 | tail -1; done
python scripts/isolated.py stencil histo bfs spmv sgemm --reps 3 --policy resolve 2>&1 | python -c "
import sys,json
for line in sys.stdin:
    t,j=line.split(' ',1); j=json.loads(j); print(t, 'ovh resolve %.3f'%(j['overhead']), 'occ', j['occ'])"
