# r02b9: place_x TMA transposer tile size / CTA size (boxes per tile x threads), config 3
O=gpurun_out/r02b9
mkdir -p $O
for i in 1 2; do
  timeout 300 python bench.py --config 3 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e > $O/base_$i.json 2> $O/base_$i.err
  python -c "import json; d=json.loads(open('$O/base_$i.json').read().strip().splitlines()[-1]); print('b4 t256', round(d['ms_per_step'],4), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])"
  for v in b2 b1 b2t128 b2s3 b4t512; do
    bash scripts/variant.sh run tp$v "--config 3 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e" $O/tp${v}_$i.json
  done
done
