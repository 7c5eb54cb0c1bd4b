OUT=gpurun_out/r02_t13; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
NT_PARITY_REPORT=$OUT/parity timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1
echo "PYTEST $(tail -1 $OUT/pytest_gpu.log)"; grep -E "^FAILED|Error" $OUT/pytest_gpu.log | head -10
for rep in 1 2; do for c in csp split stream scatter; do for f in 0 1 2; do
  timeout 300 python bench.py --config $c --fused-consumers $f --no-cpu-baseline --no-e2e --no-extras --steps 5 --json-out $OUT/f_${c}_${f}_$rep.json > /dev/null 2>&1
  python -c "import json; d=json.load(open('$OUT/f_${c}_${f}_$rep.json')); print('$rep $c fused=$f', '%.2f ms' % d['roofline']['kernel_ms'], 'frac %.3f' % d['roofline']['frac'], 'l2 %.3f' % d['l2_red_roofline']['frac'], d['clocks']['sm_mhz'])" 2>&1 | tail -1
done; done; done
for tool in memcheck racecheck; do
  timeout 1200 compute-sanitizer --tool $tool --print-limit 50 python scripts/sanitize_run.py > $OUT/sanitizer_$tool.log 2>&1
  echo "SANITIZER $tool rc=$? $(grep -E 'ERROR SUMMARY|RACECHECK SUMMARY|runs clean' $OUT/sanitizer_$tool.log | tr '\n' ' ')"
done
bash scripts/dev/ab_variants.sh r02_ab11_ev_regtypes "evbase evreg evr8" "csp:event stream:event split:event scatter:event" 2 | grep -v pytest
