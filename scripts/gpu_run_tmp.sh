timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -k "k0 or cluster or thread_level or config" 2>&1 | tail -15 > gpurun_out/t_k0.txt
P='[{"k_pass": [], "cluster": 2, "tl_levels": 2, "cr_levels": 3, "thomas_chains": 64},
{"k_pass": [], "cluster": 2, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 16},
{"k_pass": [3], "cluster": 1, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 4, "split_threads": 512}]'
timeout 300 python scripts/sweep.py --n 16384 --m 4096 --reps 10 --points "$P" > gpurun_out/sweep_c4.txt 2>&1
cat gpurun_out/t_k0.txt; python -c "
import json
for l in open('gpurun_out/sweep_c4.txt'):
    try: d=json.loads(l)
    except Exception: print(l[:300]); continue
    print(d['params'], d.get('error') or (d['stage_ms'], d['total_ms'], d['geq_per_s']))
"
