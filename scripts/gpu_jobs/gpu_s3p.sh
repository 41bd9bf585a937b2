# session 3p: eviction without a CAS loop (uniform datapath back in RESOLVE bodies)
export ACCEL_DEBUG_OFF=1
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/gpu_suite8.log 2>&1; tail -2 gpurun_out/gpu_suite8.log; grep FAILED gpurun_out/gpu_suite8.log
timeout 600 python scripts/isolated.py stencil histo bfs spmv sgemm mriq cutcp tpacf --reps 5 --policy both > gpurun_out/iso_p.log 2>&1
python - <<'PY'
import json
for line in open("gpurun_out/iso_p.log"):
    if " {" not in line: print(line[:200]); continue
    t, j = line.split(" ", 1); j = json.loads(j)
    print(t, {k: round(v, 4) for k, v in j.items() if k.startswith("overhead")}, {k: round(v["elapsed_ms"], 3) for k, v in j.items() if isinstance(v, dict)})
PY
timeout 600 python bench.py --steps 10 --warmup 3 --out gpurun_out/bench_c2.json > gpurun_out/bench_c2.log 2>&1
python - <<'PY'
import json
j = json.load(open("gpurun_out/bench_c2.json")); s = j["sharing"]
print(j["value"], j["e2e"]["value"], {k: round(s[k], 3) for k in ["unfairness_shared", "unfairness_native", "stp_shared", "stp_native", "stp_ratio", "throughput_speedup"]},
      {k: round(v, 2) for k, v in s["T_s_ms_shared"].items()}, s["other_policies"]["static"]["unfairness"], s["other_policies"]["static"]["stp"])
PY
timeout 600 ncu --set full --clock-control none --import-source on -k regex:accel_persistent -s 10 -c 1 -o gpurun_out/r1d_stencil_resolve python scripts/profile_one.py stencil resolve default sweeps=12 > /dev/null 2>&1; ls gpurun_out/r1d*
