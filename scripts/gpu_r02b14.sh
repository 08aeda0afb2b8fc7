# r02b14: the intermittent config-2 bench hang: default (e2e + cpu baseline) vs e2e only vs cpu only
O=gpurun_out/r02b14
mkdir -p $O
nproc > $O/nproc.txt; python -c "import os; print(len(os.sched_getaffinity(0)))" >> $O/nproc.txt
for i in 1 2 3; do
  for mode in default noe2e nocpu; do
    extra=""; [ $mode = noe2e ] && extra="--no-e2e"; [ $mode = nocpu ] && extra="--no-cpu-baseline"
    timeout -s ABRT 150 python -X faulthandler bench.py --config 2 --steps 50 --warmup 5 $extra > $O/${mode}_$i.json 2> $O/${mode}_$i.err
    echo "$mode $i rc=$?"
  done
done
cat $O/nproc.txt
