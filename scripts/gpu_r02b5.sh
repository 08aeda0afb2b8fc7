# r02b5: conflict-free split transpose (TR34, product) vs the swizzled [rho][m] rows (variant tr34off):
# config 3 bench x3 each, split/coupling GPU tests with the product build, ncu bank conflicts of the split
O=gpurun_out/r02b5
mkdir -p $O
for i in 1 2 3; do
  timeout 300 python bench.py --config 3 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e > $O/new_$i.json 2> $O/new_$i.err
  python -c "import json; d=json.loads(open('$O/new_$i.json').read().strip().splitlines()[-1]); print('new', round(d['ms_per_step'],4), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']], d['clocks']['reasons'])"
  bash scripts/variant.sh run tr34off "--config 3 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e" $O/old_$i.json
done
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -x -k "split or coupling or fuzz or bench or full_size" > $O/tests.txt 2>&1; tail -3 $O/tests.txt
timeout 300 ncu --metrics gpu__time_duration.sum,l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum,l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum,l1tex__data_pipe_lsu_wavefronts_mem_shared.sum,smsp__inst_executed.sum -k regex:split_pipe -c 2 python scripts/probes/split_probe.py --only 512 7 > $O/ncu_split.txt 2>&1; grep -E "split_pipe|duration|conflicts|wavefronts|inst_executed" $O/ncu_split.txt | head -14
