# session 3l: multi-launch growth by sticky top-ups vs none (C2, C4), and the C2 timeline
export ACCEL_DEBUG_OFF=1
for v in 0 1; do
  if [ $v = 1 ]; then export ACCEL_NO_MULTI_TOPUP=1; fi
  timeout 600 python bench.py --steps 10 --warmup 3 --calib-reps 3 --no-cpu-baseline --out gpurun_out/bench_nt$v.json > gpurun_out/bench_nt$v.log 2>&1
  python - $v <<'PY'
import json, sys
j = json.load(open(f"gpurun_out/bench_nt{sys.argv[1]}.json")); s = j["sharing"]
print("no_multi_topup", sys.argv[1], {k: round(s[k], 3) for k in ["unfairness_shared", "stp_ratio", "throughput_speedup"]},
      {k: round(v, 2) for k, v in s["T_s_ms_shared"].items()})
PY
  timeout 600 python scripts/mixes.py --config c4 --reps 5 --modes resolve --out gpurun_out/c4_nt$v.json > gpurun_out/c4_nt$v.log 2>&1; grep SUMMARY gpurun_out/c4_nt$v.log | python -c "import json,sys; l=sys.stdin.read(); j=json.loads(l.split('SUMMARY',1)[1]); r=j['resolve']; print('c4', {k: round(r[k],3) for k in ['U','STP','ANTT','STP_ratio','throughput_speedup']})"
done
unset ACCEL_NO_MULTI_TOPUP
timeout 120 python scripts/timeline.py resolve c2 2>&1 | tail -40
