# DEV A/B: block-map block side 32 (default at 4000^2) vs 64 vs 128 (NT_BLK_SHIFT), history + event
OUT=gpurun_out/r02_blk; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
NT_BLK_SHIFT=6 timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -q -p no:cacheprovider -x -k "production or deterministic" > $OUT/pytest.log 2>&1
echo "PYTEST(shift 6) $(tail -1 $OUT/pytest.log)"
for rep in 1 2; do
  for cm in csp:history csp:event stream:event split:event stream:history; do
    c=${cm%%:*}; m=${cm##*:}
    for v in 5 6 7; do
      NT_BLK_SHIFT=$v python bench.py --config $c --mode $m --steps 3 --warmup 3 --no-cpu-baseline --no-e2e --no-extras \
        --json-out $OUT/b_${c}_${m}_s${v}_r$rep.json > /dev/null 2>&1
      python -c "
import json; d=json.load(open('$OUT/b_${c}_${m}_s${v}_r$rep.json'))
print('$c $m shift=$v rep=$rep', 'kernel_ms %.3f' % d['roofline']['kernel_ms'])" 2>&1 | tail -1
    done
  done
done
