# resume ring A/B (round 2): parity of the ring and the default paths, then interleaved
# bench runs with resume_prefetch 0 / 1 on csp, split, scatter, stream (history mode).
TAG=${1:-r02_ring}
OUT=gpurun_out/$TAG; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -x -k "resume_prefetch or deferral or fused or smoke or xs" > $OUT/pytest.log 2>&1
echo "PYTEST $(tail -1 $OUT/pytest.log)"; grep -E "^FAILED|Error" $OUT/pytest.log | head
for rep in 1 2; do
  for c in csp split scatter stream; do
    for v in 0 1; do
      python bench.py --config $c --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --no-extras \
        --resume-prefetch $v --json-out $OUT/b_${c}_rp${v}_r$rep.json > $OUT/b_${c}_rp${v}_r$rep.log 2>&1
      python -c "
import json; d=json.load(open('$OUT/b_${c}_rp${v}_r$rep.json'))
print('$c rp=$v rep=$rep', 'kernel_ms %.3f' % d['roofline']['kernel_ms'], 'ms %.3f' % d['ms_per_step'])" 2>&1 | tail -1
    done
  done
done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:history -c 2 -o $OUT/prof_csp_ring \
  python bench.py --config csp --steps 1 --warmup 0 --no-cpu-baseline --no-e2e --no-extras --resume-prefetch 1 > $OUT/ncu_ring.log 2>&1
python scripts/ncu_summary.py $OUT/prof_csp_ring.ncu-rep $OUT/ncu_csp_ring.md > /dev/null 2>&1
rm -f $OUT/prof_csp_ring.ncu-rep
python bench.py --steps 5 --warmup 3 --no-cpu-baseline --no-extras --json-out $OUT/b_e2e.json > $OUT/b_e2e.log 2>&1
python -c "
import json; d=json.load(open('$OUT/b_e2e.json')); print('E2E', d['value'], d['ms_per_step'], d['e2e']['value'], d['e2e']['ms_per_step'])"
