# r02b21: on-chip warp form, early operation order on the serial path (variant serearly) vs product, config 3
O=gpurun_out/r02b21
mkdir -p $O
for i in 1 2 3; do
  timeout 300 python bench.py --config 3 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e > $O/base_$i.json 2> $O/base_$i.err
  python -c "import json; d=json.loads(open('$O/base_$i.json').read().strip().splitlines()[-1]); print('product', round(d['ms_per_step'],5), [(k['kernel'], round(k['ms'],5)) for k in d['roofline']['per_kernel']])"
  bash scripts/variant.sh run serearly "--config 3 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e" $O/ser_$i.json
done
