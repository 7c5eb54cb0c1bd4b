OUT=gpurun_out/r02_t12; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
NT_PARITY_REPORT=$OUT/parity timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1
echo "PYTEST $(tail -1 $OUT/pytest_gpu.log)"; grep -E "^FAILED|Error" $OUT/pytest_gpu.log | head -10
bash scripts/dev/ab_variants.sh r02_ab10_ev_refill "evr16 evr8 evr32" "csp:event stream:event split:event scatter:event" 2 | grep -v pytest
timeout 900 ncu --set full --clock-control none --import-source on -k regex:ev_loop -c 1 -o $OUT/prof_csp_event python bench.py --config csp --mode event --steps 1 --warmup 0 --no-cpu-baseline --no-e2e --no-extras > $OUT/ncu_csp_event.log 2>&1
python scripts/ncu_summary.py $OUT/prof_csp_event.ncu-rep $OUT/ncu_csp_event.md > /dev/null 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:history -c 1 -o $OUT/prof_scatter_history python bench.py --config scatter --steps 1 --warmup 0 --no-cpu-baseline --no-e2e --no-extras > $OUT/ncu_scatter.log 2>&1
python scripts/ncu_summary.py $OUT/prof_scatter_history.ncu-rep $OUT/ncu_scatter_history.md > /dev/null 2>&1
rm -f $OUT/*.ncu-rep
