# A/B: fused phases with tail mixing (fused_consumers k: k-1 dedicated consumer CTAs per SM,
# every producer warp resumes parked particles once the range is exhausted) vs two launches.
TAG=${1:-r02_fz2}
OUT=gpurun_out/$TAG; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -x -k "fused or xs or smoke" > $OUT/pytest.log 2>&1
echo "PYTEST $(tail -1 $OUT/pytest.log)"; grep -E "^FAILED|Error" $OUT/pytest.log | head -5
for rep in 1 2; do
  for c in csp split scatter stream; do
    for f in 0 1 2; do
      python bench.py --config $c --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --no-extras \
        --fused-consumers $f --json-out $OUT/b_${c}_f${f}_r$rep.json > $OUT/b_${c}_f${f}_r$rep.log 2>&1
      python -c "
import json; d=json.load(open('$OUT/b_${c}_f${f}_r$rep.json'))
print('$c fused=$f rep=$rep', 'kernel_ms %.3f' % d['roofline']['kernel_ms'])" 2>&1 | tail -1
    done
  done
done
python bench.py --steps 5 --warmup 3 --no-cpu-baseline --no-extras --json-out $OUT/b_e2e.json > $OUT/b_e2e.log 2>&1
python -c "
import json; d=json.load(open('$OUT/b_e2e.json')); print('E2E', d['value'], d['ms_per_step'], d['e2e']['value'], d['e2e']['ms_per_step'])"
