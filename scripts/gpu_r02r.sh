mkdir -p gpurun_out/r02r
O=gpurun_out/r02r
python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.txt 2>&1; cat $O/smoke.txt
timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider -rfs > $O/gputests.txt 2>&1
tail -3 $O/gputests.txt
timeout 300 python scripts/sanitize.py > $O/san_plain.txt 2>&1; tail -3 $O/san_plain.txt
for tool in memcheck racecheck synccheck; do
  timeout 1500 compute-sanitizer --tool $tool --print-limit 20 python scripts/sanitize.py > $O/san_$tool.txt 2>&1
  echo "== $tool rc=$?"; grep -E "SUMMARY|BAD" $O/san_$tool.txt | head -5; grep -c "^ok" $O/san_$tool.txt
done
