OUT=gpurun_out/r02_fma; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
bash scripts/dev/build_variants.sh "fmad:-fmad=true" "nofma:" > /dev/null 2>&1
NT_LIB_VARIANT=fmad python scripts/dev/fma_flip_rate.py > $OUT/flip_fmad.log 2>&1; tail -1 $OUT/flip_fmad.log > $OUT/flip_fmad.json; grep -v "^{" $OUT/flip_fmad.log | cut -c1-200
for rep in 1 2; do for cm in scatter:history csp:history split:history scatter:event csp:event; do for v in nofma fmad; do
  c=${cm%%:*}; m=${cm##*:}
  NT_LIB_VARIANT=$v timeout 300 python bench.py --config $c --mode $m --no-cpu-baseline --no-e2e --no-extras --steps 5 --json-out $OUT/t.json > /dev/null 2>&1
  python -c "import json; d=json.load(open('$OUT/t.json')); print('$rep $c $m $v', '%.2f ms' % d['roofline']['kernel_ms'], d['clocks']['sm_mhz'])" 2>&1 | tail -1
done; done; done
