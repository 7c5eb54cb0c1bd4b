# A/B: unionised grid (xs_search 4) vs direct rows (0); parity of the XS paths first
OUT=gpurun_out/r02_ug; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -x -k "xs or smoke" > $OUT/pytest.log 2>&1
echo "PYTEST $(tail -1 $OUT/pytest.log)"; grep -E "^FAILED" $OUT/pytest.log | head -5
for rep in 1 2; do
  for cm in scatter:history scatter:event csp:history csp:event split:history; do
    c=${cm%%:*}; m=${cm##*:}
    for x in 0 4; do
      python bench.py --config $c --mode $m --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --no-extras --xs-search $x \
        --json-out $OUT/b_${c}_${m}_xs${x}_r$rep.json > /dev/null 2>&1
      python -c "
import json; d=json.load(open('$OUT/b_${c}_${m}_xs${x}_r$rep.json'))
print('$c $m xs=$x rep=$rep', 'kernel_ms %.3f' % d['roofline']['kernel_ms'])" 2>&1 | tail -1
    done
  done
done
