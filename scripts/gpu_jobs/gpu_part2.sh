# LPT dequeue order (cutcp, tpacf) + partition fixes: GPU suite, isolated overhead, C2 bench
timeout 1500 python -m pytest tests -m gpu -x -q 2>&1 | tail -8
timeout 600 python scripts/isolated.py cutcp tpacf stencil spmv sgemm mriq --reps 3 --policy all > gpurun_out/iso_part2.log 2>&1
python - <<'PY'
import json
for line in open("gpurun_out/iso_part2.log"):
    if " {" not in line: print(line[:300]); continue
    t, j = line.split(" ", 1); j = json.loads(j)
    print(t, {k: round(v, 3) for k, v in j.items() if k.startswith("overhead")}, {k: round(v["elapsed_ms"], 3) for k, v in j.items() if isinstance(v, dict)})
PY
timeout 900 python bench.py --steps 5 --warmup 3 --calib-reps 3 --policy resolve --no-cpu-baseline --out gpurun_out/bench_lpt.json > gpurun_out/bench_lpt.log 2>&1; tail -c 300 gpurun_out/bench_lpt.log
timeout 900 python scripts/mixes.py --config c3 --tenants mriq,cutcp,sgemm,histo,stencil,tpacf --only mriq:mriq,cutcp:sgemm,histo:mriq,cutcp:cutcp,stencil:histo,tpacf:tpacf,sgemm:stencil,cutcp:stencil --reps 2 --out gpurun_out/pairs_part.json 2>&1 | tail -12
