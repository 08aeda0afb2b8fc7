mkdir -p gpurun_out/r02f
O=gpurun_out/r02f
timeout 300 python scripts/sanitize.py > $O/san_plain.txt 2>&1; tail -5 $O/san_plain.txt
for tool in memcheck racecheck synccheck; do
  timeout 1500 compute-sanitizer --tool $tool --print-limit 20 python scripts/sanitize.py > $O/san_$tool.txt 2>&1
  echo "== $tool rc=$?"; grep -E "SUMMARY|BAD" $O/san_$tool.txt | head -20; grep -c "^ok" $O/san_$tool.txt
done
timeout 2400 python scripts/fuzz_long.py 3000 11 > $O/fuzz.txt 2>&1; echo "fuzz rc=$?"; tail -5 $O/fuzz.txt
