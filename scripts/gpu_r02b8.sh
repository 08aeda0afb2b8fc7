# r02b8: place_x TMA transposer pipeline depth (input stages x output buffers), config 3
O=gpurun_out/r02b8
mkdir -p $O
for i in 1 2; do
  timeout 300 python bench.py --config 3 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e > $O/base_$i.json 2> $O/base_$i.err
  python -c "import json; d=json.loads(open('$O/base_$i.json').read().strip().splitlines()[-1]); print('tp21', round(d['ms_per_step'],4), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])"
  for v in 31 22 32 42 41; do
    bash scripts/variant.sh run tp$v "--config 3 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e" $O/tp${v}_$i.json
  done
done
