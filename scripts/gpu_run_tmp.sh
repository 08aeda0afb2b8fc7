timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -k "stride or isolation" 2>&1 | tail -8
