# compute-sanitizer over every kernel family (scripts/sanitize.py); summaries to gpurun_out/
timeout 300 python scripts/sanitize.py > gpurun_out/san_plain.txt 2>&1; tail -20 gpurun_out/san_plain.txt
for tool in memcheck racecheck synccheck; do  # initcheck: TMA stores are not tracked (false "uninitialized" on x)
  timeout 1500 compute-sanitizer --tool $tool --print-limit 20 python scripts/sanitize.py > gpurun_out/san_$tool.txt 2>&1
  echo "== $tool rc=$?"; grep -E "SUMMARY|BAD|^ok" gpurun_out/san_$tool.txt | head -20
done
