# session 3x: dequeue order experiment for the issue-bound tenants (isolated, both policies)
export ACCEL_DEBUG_OFF=1
for o in lpt linear zigzag lpt_tail:0.5 lpt_tail:0.3; do
  ACCEL_ORDER_EXPERIMENT=$o timeout 300 python scripts/isolated.py cutcp tpacf --reps 5 --policy both > gpurun_out/ord.log 2>&1
  python - "$o" <<'PY'
import json, sys
for line in open("gpurun_out/ord.log"):
    if " {" not in line: continue
    t, j = line.split(" ", 1); j = json.loads(j)
    print(sys.argv[1], t, {k: round(v, 4) for k, v in j.items() if k.startswith("overhead")})
PY
done
