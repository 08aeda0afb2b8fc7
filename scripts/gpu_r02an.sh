# fp64 row update in the early order (-DTDS_FP64_EARLY=1) vs the product order, config 3 fp64 + fp64 tests
O=gpurun_out/r02an
mkdir -p $O
for i in 1 2 3; do
  timeout 300 python bench.py --config 3 --dtype f64 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e > $O/base_$i.json 2> $O/base_$i.err
  python -c "import json; d=json.loads(open('$O/base_$i.json').read().strip().splitlines()[-1]); print('base', round(d['ms_per_step'],4), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']], d['clocks']['reasons'])"
  bash scripts/variant.sh run f64early "--config 3 --dtype f64 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e" $O/early_$i.json
done
W=/tmp/tds_var_f64early
(cd $W && timeout 1200 python -m pytest tests -m gpu -q -p no:cacheprovider -k "float64 or f64 or coupling or F64" -x > /root/repo/$O/tests_early.txt 2>&1); tail -3 $O/tests_early.txt
