# r02b12: config-2 bench reproduction (r02fin4 timed out at 900 s with no output)
O=gpurun_out/r02b12
mkdir -p $O
for i in 1 2; do
  timeout 240 python -X faulthandler bench.py --config 2 --steps 50 --warmup 5 --tune-cache $O/tune.txt > $O/cfg2_$i.json 2> $O/cfg2_$i.err
  echo "rc=$?"; head -c 400 $O/cfg2_$i.json; echo; tail -3 $O/cfg2_$i.err
done
cat $O/tune.txt
