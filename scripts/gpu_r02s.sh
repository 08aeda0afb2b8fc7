mkdir -p gpurun_out/r02s
O=gpurun_out/r02s
timeout 1500 python -m pytest tests/test_dist.py -m gpu -q -p no:cacheprovider -rf > $O/tests.txt 2>&1; tail -5 $O/tests.txt
timeout 300 python bench.py --steps 20 --warmup 3 --no-cpu-baseline --no-e2e --tune-cache /tmp/c3.tune > $O/cfg3.json 2> $O/cfg3.err
python -c "import json; d=json.loads(open('$O/cfg3.json').read().strip().splitlines()[-1]); print('cfg3', round(d['ms_per_step'],4), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])"
