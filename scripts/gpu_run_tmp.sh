P='[{"k_pass": [7], "cluster": 1, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 16}]'
timeout 300 ncu --set full --clock-control none --import-source on -s 3 -c 3 -o gpurun_out/prof_cur python scripts/sweep.py --n 1048576 --m 16 --reps 1 --points "$P" > /dev/null 2>&1
ls gpurun_out
