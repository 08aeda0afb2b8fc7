# r02b17: conflict-free sub-row transpose for the fp64 256-thread split (product) vs the
# swizzled rows (notr34: both dtypes off); fp64 + coupling + split GPU tests
O=gpurun_out/r02b17
mkdir -p $O
for i in 1 2 3; do
  timeout 300 python bench.py --config 3 --dtype f64 --steps 30 --warmup 5 --no-cpu-baseline --no-e2e > $O/new_$i.json 2> $O/new_$i.err
  python -c "import json; d=json.loads(open('$O/new_$i.json').read().strip().splitlines()[-1]); print('new', round(d['ms_per_step'],4), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']], d['clocks']['reasons'])"
  bash scripts/variant.sh run notr34 "--config 3 --dtype f64 --steps 30 --warmup 5 --no-cpu-baseline --no-e2e" $O/old_$i.json
done
timeout 1200 python -m pytest tests -m gpu -q -p no:cacheprovider -k "f64 or float64 or coupling or split or fuzz or full_size or huge" > $O/tests.txt 2>&1; tail -3 $O/tests.txt
timeout 300 ncu --metrics gpu__time_duration.sum,l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum,l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum -k regex:split_pipe -c 1 python bench.py --config 3 --dtype f64 --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline --mode static > $O/ncu.txt 2>&1; grep -E "conflicts|duration" $O/ncu.txt
