# DEV A/B: phase 2 with the 72-register kernel at 7 CTAs/SM (NT_P2_MINB=7) vs the default
OUT=gpurun_out/r02_p2m; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
NT_P2_MINB=7 timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -q -p no:cacheprovider -x -k "production or deferral or resume" > $OUT/pytest.log 2>&1
echo "PYTEST(p2 minb 7) $(tail -1 $OUT/pytest.log)"
for rep in 1 2; do
  for c in csp split scatter stream; do
    for v in 0 7; do
      if [ $v = 0 ]; then unset NT_P2_MINB; else export NT_P2_MINB=$v; fi
      python bench.py --config $c --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --no-extras \
        --json-out $OUT/b_${c}_m${v}_r$rep.json > /dev/null 2>&1
      python -c "
import json; d=json.load(open('$OUT/b_${c}_m${v}_r$rep.json'))
print('$c p2minb=$v rep=$rep', 'kernel_ms %.3f' % d['roofline']['kernel_ms'])" 2>&1 | tail -1
    done
  done
done
unset NT_P2_MINB
