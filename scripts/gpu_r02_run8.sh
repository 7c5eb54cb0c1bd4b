OUT=gpurun_out/r02_t8; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
NT_PARITY_REPORT=$OUT/parity timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1
echo "PYTEST $(tail -1 $OUT/pytest_gpu.log)"; grep -E "^FAILED|Error" $OUT/pytest_gpu.log | head -10
for c in csp stream split scatter; do
  timeout 300 python bench.py --config $c --mode event --no-cpu-baseline --no-e2e --no-extras --steps 5 --json-out $OUT/b_${c}_event.json > /dev/null 2>&1
  python -c "import json; d=json.load(open('$OUT/b_${c}_event.json')); print('$c event', '%.2f ms' % d['roofline']['kernel_ms'], 'frac %.3f' % d['roofline']['frac'], d['clocks']['sm_mhz'])" 2>&1 | tail -1
done
for rep in 1 2; do
 for c in scatter_src001 scatter csp; do for t in 0 1 2 3; do
  timeout 300 python bench.py --config $c --tally-mode $t --no-cpu-baseline --no-e2e --no-extras --steps 5 --json-out $OUT/t_${c}_${t}_$rep.json > /dev/null 2>&1
  python -c "import json; d=json.load(open('$OUT/t_${c}_${t}_$rep.json')); print('$rep tally', '$c', 'mode=$t', '%.2f ms' % d['roofline']['kernel_ms'], d['clocks']['sm_mhz'])" 2>&1 | tail -1
 done; done
 for c in csp scatter split; do for l in 0 1; do
  timeout 300 python bench.py --config $c --particle-layout $l --no-cpu-baseline --no-e2e --no-extras --steps 5 --json-out $OUT/l_${c}_${l}_$rep.json > /dev/null 2>&1
  python -c "import json; d=json.load(open('$OUT/l_${c}_${l}_$rep.json')); print('$rep layout', '$c', 'aos=$l', '%.2f ms' % d['roofline']['kernel_ms'], d['clocks']['sm_mhz'])" 2>&1 | tail -1
 done; done
done
for tool in memcheck racecheck synccheck initcheck; do
  timeout 1200 compute-sanitizer --tool $tool --print-limit 50 python scripts/sanitize_run.py > $OUT/sanitizer_$tool.log 2>&1
  echo "SANITIZER $tool rc=$? $(grep -E 'ERROR SUMMARY|runs clean' $OUT/sanitizer_$tool.log | tr '\n' ' ')"
done
