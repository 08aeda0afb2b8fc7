# GPU parity suite + a sweep of the config-3 candidate plans (per-kernel ms, back-to-back total)
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -x -q 2>&1 | tail -2 > gpurun_out/t_all.txt
P=${SWEEP_POINTS:-'[{"k_pass": [7], "cluster": 1, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 16},
{"k_pass": [8], "cluster": 1, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 8},
{"k_pass": [6], "cluster": 2, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 16},
{"k_pass": [5], "cluster": 2, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 16}]'}
timeout 300 python scripts/sweep.py --n 1048576 --m 16 --reps 20 --points "$P" > gpurun_out/sweep_a.txt 2>&1
cat gpurun_out/t_all.txt; python -c "
import json
for l in open('gpurun_out/sweep_a.txt'):
    d=json.loads(l)
    print(d['params'], d.get('error') or (d['stage_ms'], d['total_ms'], d['geq_per_s']))
"
