timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -x -q 2>&1 | tail -2 > gpurun_out/t_all.txt
P='[{"k_pass": [8], "cluster": 1, "tl_levels": 5, "cr_levels": 3, "thomas_chains": 16},
{"k_pass": [4,4], "cluster": 1, "tl_levels": 5, "cr_levels": 3, "thomas_chains": 16},
{"k_pass": [5,3], "cluster": 1, "tl_levels": 5, "cr_levels": 3, "thomas_chains": 16}]'
timeout 300 python scripts/sweep.py --dtype float64 --n 1048576 --m 16 --reps 10 --points "$P" > gpurun_out/sweep_f64.txt 2>&1
cat gpurun_out/t_all.txt; python -c "
import json
for l in open('gpurun_out/sweep_f64.txt'):
    try: d=json.loads(l)
    except Exception: print(l[:300]); continue
    print(d['params'], d.get('error') or (d['stage_ms'], d['total_ms'], d['geq_per_s']))
"
