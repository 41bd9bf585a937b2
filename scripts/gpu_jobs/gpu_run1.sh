set -x
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
python -c "import torch; print(torch.cuda.get_device_name())"
timeout 900 python -m pytest tests -m gpu -x -q 2>&1 | tail -30
timeout 300 python __graft_entry__.py smoke 2>&1 | tail -5
timeout 300 python scripts/isolated.py stencil histo mop 2>&1 | tail -5
timeout 600 python bench.py --config c1 --steps 5 --warmup 3 --out gpurun_out/bench_c1.json 2>&1 | tail -5
