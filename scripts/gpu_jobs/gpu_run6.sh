timeout 1500 python -m pytest tests -m gpu -q 2>&1 | tail -25
timeout 600 python scripts/isolated.py spmv sgemm mriq bfs 2>&1 | tail -4
