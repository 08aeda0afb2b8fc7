python bench.py --steps 30 --warmup 3 --no-cpu-baseline --no-e2e 2>&1 | tail -1 | python -c "
import json,sys; d=json.loads(sys.stdin.read()); print(d['value'], d['ms_per_step'], d['config']['plan'], d['config']['tune_trials'], d['config']['tune_s']); print(json.dumps(d['roofline']['per_kernel']))"
