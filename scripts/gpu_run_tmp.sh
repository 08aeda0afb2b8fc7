timeout 300 python bench.py --steps 30 --warmup 5 --no-e2e --no-cpu-baseline --soak-s 0 --tune-cache gpurun_out/tc.txt > gpurun_out/pdl3.json 2>gpurun_out/pdl3.err
for c in 2 4; do timeout 300 python bench.py --config $c --steps 30 --warmup 5 --no-e2e --no-cpu-baseline --soak-s 0 > gpurun_out/pdl$c.json 2>gpurun_out/pdl$c.err; done
for c in 3 2 4; do python -c "
import json; d=json.load(open('gpurun_out/pdl$c.json')); print($c, round(d['ms_per_step'],4), '%.3e'%d['value'], [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])"; done
timeout 1200 python -m pytest tests -m gpu -x -q -p no:cacheprovider 2>&1 | tail -3
