timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -k "k0 or cluster or inplace or isolation or config" 2>&1 | tail -3 > gpurun_out/t_k0.txt
P='[{"k_pass": [], "cluster": 8, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 16}, {"k_pass": [], "cluster": 4, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 16}]'
timeout 300 python scripts/sweep.py --n 65536 --m 256 --reps 10 --points "$P" > gpurun_out/sweep_c2.txt 2>&1
P='[{"k_pass": [], "cluster": 2, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 16}]'
timeout 300 python scripts/sweep.py --n 16384 --m 4096 --reps 10 --points "$P" >> gpurun_out/sweep_c2.txt 2>&1
cat gpurun_out/t_k0.txt; python -c "
import json
for l in open('gpurun_out/sweep_c2.txt'):
    try: d=json.loads(l)
    except Exception: print(l[:300]); continue
    print(d['params'], d.get('error') or (d['stage_ms'], d['total_ms'], d['geq_per_s']))
"
