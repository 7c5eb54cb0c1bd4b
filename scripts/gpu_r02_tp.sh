# DEV A/B: tail parking (NT_TAIL_PARK = lanes) in phase 1; e2e per-call events
TAG=${1:-r02_tp}
OUT=gpurun_out/$TAG; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
python scripts/dev/e2e_events.py csp > $OUT/e2e_events.json 2> $OUT/e2e_events.err; tail -1 $OUT/e2e_events.json
NT_TAIL_PARK=16 timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -p no:cacheprovider -x -k "deferral or resume_prefetch or parity_config or two_steps" > $OUT/pytest.log 2>&1
echo "PYTEST(tail 16) $(tail -1 $OUT/pytest.log)"
for rep in 1 2; do
  for c in csp split stream scatter; do
    for v in 0 8 16 24; do
      NT_TAIL_PARK=$v python bench.py --config $c --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --no-extras \
        --json-out $OUT/b_${c}_tp${v}_r$rep.json > /dev/null 2>&1
      python -c "
import json; d=json.load(open('$OUT/b_${c}_tp${v}_r$rep.json'))
print('$c tail_park=$v rep=$rep', 'kernel_ms %.3f' % d['roofline']['kernel_ms'])" 2>&1 | tail -1
    done
  done
done
