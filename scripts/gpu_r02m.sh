mkdir -p gpurun_out/r02m
O=gpurun_out/r02m
for m in 2 4 16; do
  for i in 1 2; do
    bash scripts/variant.sh run pdl "--config 3 --systems $m --launch graph --steps 50 --warmup 5 --no-e2e --no-cpu-baseline --tune-cache /tmp/c3_$m.tune" $O/var_pdl_m${m}_$i.json
    timeout 600 python bench.py --config 3 --systems $m --launch graph --steps 50 --warmup 5 --no-e2e --no-cpu-baseline --tune-cache /tmp/c3_$m.tune > $O/base_m${m}_$i.json 2> $O/base_m${m}_$i.err
    python -c "import json; d=json.loads(open('$O/base_m${m}_$i.json').read().strip().splitlines()[-1]); print('base m=$m', round(d['ms_per_step'],4))"
  done
done
for m in 4096 512; do
  bash scripts/variant.sh run pdl "--config 4 --systems $m --launch graph --steps 50 --warmup 5 --no-e2e --no-cpu-baseline --tune-cache /tmp/c4_$m.tune" $O/var_pdl_c4m${m}.json
  timeout 600 python bench.py --config 4 --systems $m --launch graph --steps 50 --warmup 5 --no-e2e --no-cpu-baseline --tune-cache /tmp/c4_$m.tune > $O/base_c4m${m}.json 2> $O/base_c4m${m}.err
  python -c "import json; d=json.loads(open('$O/base_c4m${m}.json').read().strip().splitlines()[-1]); print('base c4 m=$m', round(d['ms_per_step'],4))"
done
bash scripts/variant.sh run pdl "--config 3 --steps 50 --warmup 5 --no-e2e --no-cpu-baseline --tune-cache /tmp/c3_16.tune" $O/var_pdl_eager.json
timeout 600 python bench.py --config 3 --steps 50 --warmup 5 --no-e2e --no-cpu-baseline --tune-cache /tmp/c3_16.tune > $O/base_eager.json 2> $O/base_eager.err
python -c "import json; d=json.loads(open('$O/base_eager.json').read().strip().splitlines()[-1]); print('base eager m=16', round(d['ms_per_step'],4))"
W=/tmp/tds_var_pdl
(cd $W && timeout 1200 python -m pytest tests -m gpu -q -p no:cacheprovider -o addopts="" -x 2>&1 | tail -3) > $O/var_pdl_tests.txt
cat $O/var_pdl_tests.txt
