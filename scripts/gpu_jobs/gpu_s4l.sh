# tpacf: shared-memory RED for the lane-private bin counters (TPACF_REDS=1) vs load/add/store
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
for rd in 1 0; do
  ACCEL_NVCC_EXTRA="-DTPACF_REDS=$rd" python -m paper_conf_cgo_margiolaso16_b200.build --force > /dev/null 2>&1 || echo "build fail"
  echo "reds=$rd"
  timeout 600 python -m pytest tests -m gpu -q -x -k "tpacf" 2>&1 | tail -1
  timeout 120 python scripts/isolated.py tpacf --reps 5 2>&1 | python -c "
import sys,json
for l in sys.stdin:
  if l.startswith('tpacf'): d=json.loads(l[6:]); print('  isolated native %.3f pers %.3f res %.3f ovh %.3f regs %s occ %s' % (d['native']['elapsed_ms'], d['persistent']['elapsed_ms'], d['persistent_resolve']['elapsed_ms'], d['overhead'], d['regs'], d['occ']))"
done
