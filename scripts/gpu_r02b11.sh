# r02b11: place_x 2-box / 128-thread tiles (product) vs 4-box / 256-thread (tpold): configs 3 f32/f64, 5; GPU tests
O=gpurun_out/r02b11
mkdir -p $O
for c in "3 f32" "3 f64" "5 f32"; do
  set -- $c
  for i in 1 2; do
    timeout 300 python bench.py --config $1 --dtype $2 --steps 30 --warmup 5 --no-cpu-baseline --no-e2e > $O/new_$1$2_$i.json 2> $O/new_$1$2_$i.err
    python -c "import json; d=json.loads(open('$O/new_$1$2_$i.json').read().strip().splitlines()[-1]); print('new $1 $2', round(d['ms_per_step'],4), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])"
    bash scripts/variant.sh run tpold "--config $1 --dtype $2 --steps 30 --warmup 5 --no-cpu-baseline --no-e2e" $O/old_$1$2_$i.json
  done
done
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider > $O/gpu_tests.txt 2>&1; tail -3 $O/gpu_tests.txt
