# phase-3 A/B (defer_facets_below) on csp/split history; ncu of csp event with smem metrics
OUT=gpurun_out/r02_t5; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -p no:cacheprovider -k "deferral or deterministic" > $OUT/pytest.log 2>&1; echo "PYTEST $(tail -1 $OUT/pytest.log)"
for rep in 1 2; do for c in csp split stream; do for d in 1 4 8 16; do
  timeout 300 python bench.py --config $c --defer-facets-below $d --no-cpu-baseline --no-e2e --no-extras --steps 5 --json-out $OUT/b_${c}_$d_$rep.json > /dev/null 2>&1
  python -c "import json; d=json.load(open('$OUT/b_${c}_$d_$rep.json')); print('$rep $c dfb=$d', '%.2f ms' % d['roofline']['kernel_ms'], 'frac %.3f' % d['roofline']['frac'], d['clocks']['sm_mhz'])" 2>&1 | tail -1
done; done; done
timeout 900 ncu --set full --clock-control none --import-source on -k regex:ev_loop -c 1 -o $OUT/prof_csp_event python bench.py --config csp --mode event --steps 1 --warmup 0 --no-cpu-baseline --no-e2e --no-extras > $OUT/ncu_csp_event.log 2>&1
python scripts/ncu_summary.py $OUT/prof_csp_event.ncu-rep $OUT/ncu_csp_event.md > /dev/null 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:history -c 3 -o $OUT/prof_csp_history python bench.py --config csp --defer-facets-below 8 --steps 1 --warmup 0 --no-cpu-baseline --no-e2e --no-extras > $OUT/ncu_csp_history.log 2>&1
python scripts/ncu_summary.py $OUT/prof_csp_history.ncu-rep $OUT/ncu_csp_history.md > /dev/null 2>&1
ls -la $OUT/*.ncu-rep
rm -f $OUT/prof_csp_history.ncu-rep
