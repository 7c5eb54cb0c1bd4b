OUT=gpurun_out/r02_t10; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
NT_PARITY_REPORT=$OUT/parity timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1
echo "PYTEST $(tail -1 $OUT/pytest_gpu.log)"; grep -E "^FAILED|Error" $OUT/pytest_gpu.log | head -10
for c in csp stream split scatter; do
  timeout 300 python bench.py --config $c --mode event --no-cpu-baseline --no-e2e --no-extras --steps 5 --json-out $OUT/b_${c}_event.json > /dev/null 2>&1
  python -c "import json; d=json.load(open('$OUT/b_${c}_event.json')); print('$c event', '%.2f ms' % d['roofline']['kernel_ms'], 'frac %.3f' % d['roofline']['frac'], d['clocks']['sm_mhz'])" 2>&1 | tail -1
done
python scripts/dev/e2e_breakdown.py csp > $OUT/e2e_breakdown.json 2>&1; tail -3 $OUT/e2e_breakdown.json
bash scripts/dev/ab_variants.sh r02_ab8_early "hearly hbase" "csp:history stream:history split:history scatter:history" 2 | grep -v pytest
