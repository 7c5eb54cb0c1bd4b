# compute-sanitizer on the final tree: memcheck, racecheck, synccheck, initcheck
OUT=gpurun_out/r02_san; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
for tool in memcheck racecheck synccheck initcheck; do
  timeout 1500 compute-sanitizer --tool $tool --print-limit 50 python scripts/sanitize_run.py > $OUT/sanitizer_$tool.log 2>&1
  echo "$tool rc=$? $(grep -E 'ERROR SUMMARY|runs clean' $OUT/sanitizer_$tool.log | tr '\n' ' ')"
done
