# session 3n: round evidence -- suite, smoke, bench line, isolated overhead, C3, C4, f1 weights, ncu
export ACCEL_DEBUG_OFF=1
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/gpu_suite7.log 2>&1; tail -2 gpurun_out/gpu_suite7.log; grep FAILED gpurun_out/gpu_suite7.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -2
timeout 600 python bench.py --steps 10 --warmup 3 --out gpurun_out/bench_c2.json > gpurun_out/bench_c2.log 2>&1
python - <<'PY'
import json
j = json.load(open("gpurun_out/bench_c2.json")); s = j["sharing"]
print(j["value"], j["e2e"]["value"], {k: round(s[k], 3) for k in ["unfairness_shared", "unfairness_native", "stp_shared", "stp_native", "stp_ratio", "throughput_speedup"]},
      {k: round(v, 2) for k, v in s["T_s_ms_shared"].items()})
PY
timeout 600 python scripts/isolated.py stencil histo bfs spmv sgemm mriq cutcp tpacf --reps 5 --policy both > gpurun_out/iso_final.log 2>&1
python - <<'PY'
import json
for line in open("gpurun_out/iso_final.log"):
    if " {" not in line: print(line[:200]); continue
    t, j = line.split(" ", 1); j = json.loads(j)
    print(t, {k: round(v, 4) for k, v in j.items() if k.startswith("overhead")}, {k: round(v["elapsed_ms"], 3) for k, v in j.items() if isinstance(v, dict)})
PY
timeout 900 python scripts/mixes.py --config c3 --reps 3 --modes resolve,static --out gpurun_out/c3_pairs.json > gpurun_out/c3.log 2>&1; grep SUMMARY gpurun_out/c3.log | cut -c1-400
timeout 600 python scripts/mixes.py --config c4 --reps 5 --modes resolve,static --out gpurun_out/c4.json > gpurun_out/c4.log 2>&1; grep SUMMARY gpurun_out/c4.log | cut -c1-300
timeout 900 python scripts/weights.py --reps 5 --grid 3 --out gpurun_out/weights_c2.json > gpurun_out/weights_c2.log 2>&1; head -8 gpurun_out/weights_c2.log | cut -c1-200
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 800 --csv --log-file gpurun_out/launches_c2.csv python bench.py --steps 2 --warmup 3 --calib-reps 1 --no-cpu-baseline > gpurun_out/ncu_launch_bench.log 2>&1
NCU="timeout 600 ncu --set full --clock-control none --import-source on"
$NCU -k regex:accel_persistent -s 10 -c 1 -o gpurun_out/r1c_stencil_resolve python scripts/profile_one.py stencil resolve default sweeps=12 > /dev/null 2>&1
$NCU -k regex:accel_persistent -s 10 -c 1 -o gpurun_out/r1c_stencil_static python scripts/profile_one.py stencil persistent default sweeps=12 > /dev/null 2>&1
$NCU -k regex:accel_native -s 10 -c 1 -o gpurun_out/r1c_stencil_native python scripts/profile_one.py stencil native default sweeps=12 > /dev/null 2>&1
ls gpurun_out/r1c_*
