P='[{"k_pass": [7], "cluster": 1, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 16, "split_threads": 512},
{"k_pass": [8], "cluster": 1, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 8, "split_threads": 512}]'
SWEEP_POINTS="$P" bash scripts/gpu_test_sweep.sh
