# runtime-option sweep of the history kernel on the round-2 code: collision-deferral
# threshold, refill threshold, CTAs per SM
OUT=gpurun_out/r02_tune; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
b() {  # label, config, args
  timeout 300 python bench.py --config $2 $3 --no-cpu-baseline --no-e2e --no-extras --steps 5 --json-out $OUT/t.json > /dev/null 2>&1
  python -c "import json; d=json.load(open('$OUT/t.json')); print('$1 $2', '%.2f ms' % d['roofline']['kernel_ms'], 'l2 %.3f' % d['l2_red_roofline']['frac'], d['clocks']['sm_mhz'])" 2>&1 | tail -1
}
for rep in 1 2; do
 for c in csp split stream scatter; do
  b "$rep default" $c ""
  for d in 4 12 16; do b "$rep defer_below=$d" $c "--defer-below $d"; done
  for r in 2 8; do b "$rep refill_min=$r" $c "--refill-min $r"; done
  b "$rep ctas_per_sm=7" $c "--ctas-per-sm 7"
 done
done
