timeout 1200 python -m pytest tests -m gpu -q -x 2>&1 | tail -25
for i in 1 2 3; do timeout 300 python -m pytest tests/test_gpu_resolve.py -q -x 2>&1 | tail -1; done
