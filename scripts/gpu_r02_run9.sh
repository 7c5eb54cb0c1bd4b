OUT=gpurun_out/r02_t9; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 1200 compute-sanitizer --tool initcheck --print-limit 50 python scripts/sanitize_run.py > $OUT/sanitizer_initcheck.log 2>&1
echo "SANITIZER initcheck rc=$? $(grep -E 'ERROR SUMMARY|runs clean' $OUT/sanitizer_initcheck.log | tr '\n' ' ')"
python bench.py --json-out $OUT/bench_default.json > $OUT/bench_default.log 2>&1; echo "BENCH rc=$?"; tail -c 600 $OUT/bench_default.log
timeout 900 ncu --set full --clock-control none --import-source on -k regex:ev_loop -c 1 -o $OUT/prof_csp_event python bench.py --config csp --mode event --steps 1 --warmup 0 --no-cpu-baseline --no-e2e --no-extras > $OUT/ncu_csp_event.log 2>&1
python scripts/ncu_summary.py $OUT/prof_csp_event.ncu-rep $OUT/ncu_csp_event.md > /dev/null 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:history -c 2 -o $OUT/prof_csp_history python bench.py --config csp --steps 1 --warmup 0 --no-cpu-baseline --no-e2e --no-extras > $OUT/ncu_csp_history.log 2>&1
python scripts/ncu_summary.py $OUT/prof_csp_history.ncu-rep $OUT/ncu_csp_history.md --traffic-key csp/history > /dev/null 2>&1
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file $OUT/launches_csp.csv python bench.py --steps 2 --warmup 1 --no-cpu-baseline --no-e2e --no-extras > $OUT/ncu_launch.log 2>&1
rm -f $OUT/prof_csp_history.ncu-rep
ls -la $OUT
