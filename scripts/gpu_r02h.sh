mkdir -p gpurun_out/r02h
O=gpurun_out/r02h
timeout 900 python -m pytest tests/test_dist.py -m gpu -q -p no:cacheprovider -rf > $O/tests.txt 2>&1; tail -3 $O/tests.txt
timeout 900 python bench.py --config 5 --steps 5 --warmup 3 > $O/bench_cfg5.json 2> $O/bench_cfg5.err; echo "cfg5 rc=$?"; tail -3 $O/bench_cfg5.err
python -c "import json; d=json.loads(open('$O/bench_cfg5.json').read().strip().splitlines()[-1]); print('cfg5', round(d['ms_per_step'],4), d['value'], d['roofline']['kernel'], round(d['roofline']['frac'],3), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']], d['config']['interior_residual'])"
