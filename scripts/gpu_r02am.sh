# fp64 reciprocal: cubic single-step refinement (-DTDS_RCP64_CUBIC=1) vs two Newton steps
O=gpurun_out/r02am
mkdir -p $O
./scripts/probes/rcp64_probe | tee $O/rcp64.txt
for i in 1 2; do
  for v in base rcp3; do
    if [ $v = base ]; then
      timeout 300 python bench.py --config 3 --dtype f64 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e > $O/${v}_$i.json 2> $O/${v}_$i.err
      python -c "import json; d=json.loads(open('$O/${v}_$i.json').read().strip().splitlines()[-1]); print('$v', round(d['ms_per_step'],4), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']], d['clocks']['reasons'])"
    else
      bash scripts/variant.sh run rcp3 "--config 3 --dtype f64 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e" $O/${v}_$i.json
    fi
  done
done
W=/tmp/tds_var_rcp3
(cd $W && timeout 1200 python -m pytest tests -m gpu -q -p no:cacheprovider -k "float64 or f64 or coupling or F64" -x > /root/repo/$O/tests_rcp3.txt 2>&1); tail -3 $O/tests_rcp3.txt
