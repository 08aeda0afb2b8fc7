P='[{"k_pass": [], "cluster": 2, "tl_levels": 2, "cr_levels": 3, "thomas_chains": 64},
{"k_pass": [1], "cluster": 1, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 16, "split_threads": 512},
{"k_pass": [2], "cluster": 1, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 8, "split_threads": 512},
{"k_pass": [3], "cluster": 1, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 4, "split_threads": 512},
{"k_pass": [5], "cluster": 1, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 1, "split_threads": 512}]'
timeout 300 python scripts/sweep.py --n 16384 --m 4096 --reps 10 --points "$P" > gpurun_out/sweep_c4.txt 2>&1
python -c "
import json
for l in open('gpurun_out/sweep_c4.txt'):
    d=json.loads(l)
    print(d['params']['k_pass'], d.get('error') or (d['stage_ms'], d['total_ms'], d['geq_per_s']))
"
