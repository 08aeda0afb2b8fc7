# round-2 final evidence: smoke, the whole GPU suite, bench lines + ncu of every config,
# the reference arm, the param study, cuSPARSE context, sanitizers
TAG=${1:-r02z}
mkdir -p gpurun_out/$TAG
O=gpurun_out/$TAG
python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.txt 2>&1; cat $O/smoke.txt
timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider -rfs > $O/gputests.txt 2>&1; tail -2 $O/gputests.txt
bash scripts/gpu_final.sh $TAG > $O/final.log 2>&1; echo "final rc=$?"; grep -E "rc=" $O/final.log | tr '\n' ' '; echo
timeout 900 python scripts/param_study.py --out $O/param_study > $O/param_study.log 2>&1; echo "param rc=$?"
timeout 900 python scripts/cusparse_context.py > $O/cusparse.jsonl 2> $O/cusparse.err; echo "cusparse rc=$?"
timeout 300 python scripts/sanitize.py > $O/san_plain.txt 2>&1; tail -2 $O/san_plain.txt
for tool in memcheck racecheck synccheck; do
  timeout 1500 compute-sanitizer --tool $tool --print-limit 20 python scripts/sanitize.py > $O/san_$tool.txt 2>&1
  echo "== $tool rc=$?"; grep -E "SUMMARY|BAD" $O/san_$tool.txt | head -3; grep -c "^ok" $O/san_$tool.txt
done
