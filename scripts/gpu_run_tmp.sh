set -x
timeout 1200 python -m pytest tests -m gpu -q -p no:cacheprovider 2>&1 | tail -8
bash scripts/gpu_prof.sh r01b --mode static
