mkdir -p gpurun_out/r02o
O=gpurun_out/r02o
timeout 600 compute-sanitizer --tool memcheck --print-limit 5 python -m pytest tests/test_dist.py -m gpu -q -p no:cacheprovider -x -k "split_scatter_bit_exact and 4352 and float32" > $O/san.txt 2>&1; tail -60 $O/san.txt | head -80
