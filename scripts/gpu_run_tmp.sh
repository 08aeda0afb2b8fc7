timeout 1200 python -m pytest tests -m gpu -x -q -p no:cacheprovider 2>&1 | tail -3
python scripts/sweep.py --n 1048576 --m 16 --points '[{"k_pass": [4,3], "cluster": 1, "tl_levels": 0, "cr_levels": 4, "thomas_chains": 64}, {"k_pass": [3,4], "cluster": 1, "tl_levels": 0, "cr_levels": 4, "thomas_chains": 64}]' 2>&1 | cut -c260-480
