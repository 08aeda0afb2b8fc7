mkdir -p gpurun_out/r02q
O=gpurun_out/r02q
timeout 1200 python -m pytest tests/test_dist.py -m gpu -q -p no:cacheprovider -rf > $O/tests.txt 2>&1; tail -5 $O/tests.txt
for i in 1 2; do
timeout 300 python bench.py --steps 30 --warmup 3 --no-cpu-baseline --no-e2e --tune-cache /tmp/c3.tune > $O/cfg3_$i.json 2> $O/cfg3_$i.err
python -c "import json; d=json.loads(open('$O/cfg3_$i.json').read().strip().splitlines()[-1]); print('cfg3', round(d['ms_per_step'],4), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])"
done
