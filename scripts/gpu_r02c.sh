mkdir -p gpurun_out/r02c
O=gpurun_out/r02c
timeout 900 python -m pytest tests/test_dist.py -m gpu -q -p no:cacheprovider -rf > $O/tests.txt 2>&1
tail -3 $O/tests.txt
timeout 600 python bench.py --config 4 --steps 20 --warmup 3 --no-cpu-baseline > $O/bench_cfg4.json 2> $O/bench_cfg4.err; echo "cfg4 rc=$?"
timeout 900 python bench.py --config 5 --steps 5 --warmup 3 > $O/bench_cfg5.json 2> $O/bench_cfg5.err; echo "cfg5 rc=$?"
tail -3 $O/bench_cfg5.err
for i in 1 2; do
  bash scripts/variant.sh run stg "--config 3 --steps 30 --warmup 3 --no-e2e --no-cpu-baseline --tune-cache /tmp/c3.tune" $O/var_stg_$i.json
  timeout 600 python bench.py --config 3 --steps 30 --warmup 3 --no-e2e --no-cpu-baseline --tune-cache /tmp/c3.tune > $O/var_base_$i.json 2> $O/var_base_$i.err
  python -c "import json; d=json.loads(open('$O/var_base_$i.json').read().strip().splitlines()[-1]); print('base', round(d['ms_per_step'],4), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])"
done
