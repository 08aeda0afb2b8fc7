timeout 300 python scripts/host_probe.py
timeout 300 python bench.py --config 1 --steps 200 --warmup 10 --no-e2e --no-cpu-baseline --soak-s 0 > gpurun_out/h1.json 2>/dev/null
timeout 300 python bench.py --steps 30 --warmup 5 --no-e2e --no-cpu-baseline --soak-s 0 > gpurun_out/h3.json 2>/dev/null
for c in 1 3; do python -c "
import json; d=json.load(open('gpurun_out/h$c.json')); print($c, d['ms_per_step'], '%.3e'%d['value'], [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])"; done
timeout 1200 python -m pytest tests -m gpu -x -q -p no:cacheprovider 2>&1 | tail -2
