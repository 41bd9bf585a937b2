# PARTITION policy: parity tests, targeted pairs, C2 bench, isolated overhead
export ACCEL_DEBUG_OFF=1
timeout 900 python -m pytest tests/test_gpu_partition.py -x -q 2>&1 | tail -15
timeout 600 python scripts/isolated.py stencil histo bfs spmv sgemm mriq cutcp tpacf --reps 3 --policy all > gpurun_out/iso_part.log 2>&1
python - <<'PY'
import json
for line in open("gpurun_out/iso_part.log"):
    if not line[0].isalpha() or " {" not in line: print(line[:300]); continue
    t, j = line.split(" ", 1); j = json.loads(j)
    print(t, {k: round(v, 3) for k, v in j.items() if k.startswith("overhead")}, j.get("occ"))
PY
timeout 900 python scripts/mixes.py --config c3 --tenants mriq,cutcp,sgemm,histo,stencil,tpacf --only mriq:mriq,cutcp:sgemm,histo:mriq,cutcp:cutcp,stencil:histo,tpacf:tpacf,sgemm:stencil --reps 2 --out gpurun_out/pairs_part.json 2>&1 | tail -12
timeout 900 python bench.py --steps 5 --warmup 3 --calib-reps 3 --no-cpu-baseline --out gpurun_out/bench_part.json > gpurun_out/bench_part.log 2>&1; tail -c 400 gpurun_out/bench_part.log
