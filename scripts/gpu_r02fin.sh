# Round-2 final build evidence: gpu_r02z.sh (smoke, whole GPU suite, bench lines + ncu of
# every config, reference arm, param study, cuSPARSE, sanitizers) + all seven mutants + fuzz.
TAG=${1:-r02fin}
bash scripts/gpu_r02z.sh $TAG
O=gpurun_out/$TAG
timeout 1500 bash scripts/mutation_check.sh run $O/mutation
timeout 1200 python scripts/fuzz_long.py 6000 23 > $O/fuzz.txt 2>&1; tail -2 $O/fuzz.txt
