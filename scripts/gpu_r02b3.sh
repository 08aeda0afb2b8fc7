# r02b3: full GPU test suite on the current tree + smoke
O=gpurun_out/r02b3
mkdir -p $O
python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider > $O/gpu_tests.txt 2>&1
tail -3 $O/smoke.txt; tail -15 $O/gpu_tests.txt
