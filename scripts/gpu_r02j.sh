mkdir -p gpurun_out/r02j
O=gpurun_out/r02j
for i in 1 2; do
  bash scripts/variant.sh run trc64 "--config 3 --dtype f64 --steps 20 --warmup 3 --no-e2e --no-cpu-baseline --tune-cache /tmp/c3f64.tune" $O/var_trc64_f64_$i.json
  timeout 600 python bench.py --config 3 --dtype f64 --steps 20 --warmup 3 --no-e2e --no-cpu-baseline --tune-cache /tmp/c3f64.tune > $O/base_f64_$i.json 2> $O/base_f64_$i.err
  python -c "import json; d=json.loads(open('$O/base_f64_$i.json').read().strip().splitlines()[-1]); print('base', round(d['ms_per_step'],4), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])"
done
W=/tmp/tds_var_trc64
(cd $W && timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_coupling.py -m gpu -q -p no:cacheprovider -o addopts="" -k "deep or coupling or split or bench_launch or fuzz or families" 2>&1 | tail -3) > $O/var_trc64_tests.txt
cat $O/var_trc64_tests.txt
