# session 3v: final round evidence with the current build
export ACCEL_DEBUG_OFF=1
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/gpu_suite13.log 2>&1; tail -2 gpurun_out/gpu_suite13.log; grep -E "FAILED|STUCK" gpurun_out/gpu_suite13.log | head
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
timeout 600 python bench.py --steps 10 --warmup 3 --out gpurun_out/bench_c2.json > gpurun_out/bench_c2.log 2>&1; echo "bench rc=$?"
python - <<'PY'
import json
j = json.load(open("gpurun_out/bench_c2.json")); s = j["sharing"]
print(j["value"], j["e2e"]["value"], {k: round(s[k], 3) for k in ["unfairness_shared", "unfairness_native", "stp_ratio", "throughput_speedup"]}, j["roofline"]["frac"], j["clocks"])
PY
timeout 600 python scripts/isolated.py stencil histo bfs spmv sgemm mriq cutcp tpacf --reps 5 --policy both > gpurun_out/iso_final.log 2>&1
python - <<'PY'
import json
for line in open("gpurun_out/iso_final.log"):
    if " {" not in line: continue
    t, j = line.split(" ", 1); j = json.loads(j)
    print(t, {k: round(v, 4) for k, v in j.items() if k.startswith("overhead")})
PY
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 800 --csv --log-file gpurun_out/launches_c2.csv python bench.py --steps 2 --warmup 3 --calib-reps 1 --no-cpu-baseline > gpurun_out/ncu_launch_bench.log 2>&1; echo "ncu list rc=$?"
timeout 600 ncu --set full --clock-control none --import-source on -k regex:accel_persistent -s 10 -c 1 -o gpurun_out/r1e_stencil_resolve python scripts/profile_one.py stencil resolve default sweeps=12 > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"accel_persistent<accel::SgemmTc" -s 1 -c 1 -o gpurun_out/r1e_sgemmtc_resolve python scripts/profile_one.py sgemm resolve default > /dev/null 2>&1
ls gpurun_out/r1e*
