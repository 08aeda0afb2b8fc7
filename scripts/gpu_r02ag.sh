# Round 2: the coalesced load variant (strided = 2) -- whole GPU suite, site-7
# mutant, load-variant timings, sanitizers, a randomized plan fuzz, bench lines.
O=${O:-gpurun_out/r02ag}
mkdir -p $O
timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider -rfs > $O/gputests.txt 2>&1; tail -2 $O/gputests.txt
SITES=7 timeout 900 bash scripts/mutation_check.sh run $O
timeout 900 python scripts/probes/cv_probe.py > $O/cv_probe.txt 2>&1; tail -3 $O/cv_probe.txt
timeout 300 python scripts/sanitize.py > $O/san_plain.txt 2>&1; tail -2 $O/san_plain.txt
for tool in memcheck racecheck synccheck; do
  timeout 1500 compute-sanitizer --tool $tool --print-limit 20 python scripts/sanitize.py > $O/san_$tool.txt 2>&1
  echo "== $tool rc=$?"; grep -E "SUMMARY|BAD" $O/san_$tool.txt | head -3; grep -c "^ok" $O/san_$tool.txt
done
timeout 900 python scripts/fuzz_long.py 1500 11 > $O/fuzz.txt 2>&1; tail -3 $O/fuzz.txt
for c in 3 2 4; do
  timeout 300 python bench.py --config $c --steps 20 --warmup 3 --no-cpu-baseline --no-e2e > $O/cfg$c.json 2> $O/cfg$c.err
  python -c "import json; d=json.loads(open('$O/cfg$c.json').read().strip().splitlines()[-1]); print('cfg$c', round(d['ms_per_step'],4), d['config']['plan'].get('strided'), d['config']['plan'].get('k_pass'))"
done
