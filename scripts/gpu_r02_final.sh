# the round's evidence: GPU tests (incl. full scale), smoke, default bench (+extras, cpu
# baseline, e2e), launch list, ncu --set full of csp history/event and scatter history
TAG=${1:-r02_final}
OUT=gpurun_out/$TAG; mkdir -p $OUT
nproc > $OUT/nproc.txt
python -c "import __graft_entry__ as g; g.build()"
NT_PARITY_REPORT=$OUT/parity timeout 2700 python -m pytest tests -m gpu -q -p no:cacheprovider --durations=15 > $OUT/pytest_gpu.log 2>&1
echo "PYTEST $(tail -1 $OUT/pytest_gpu.log)"; grep -E "^FAILED|Error" $OUT/pytest_gpu.log | head -10
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke.log 2>&1; echo "SMOKE rc=$?: $(tail -1 $OUT/smoke.log)"
python bench.py --json-out $OUT/bench_default.json > $OUT/bench_default.log 2>&1; echo "BENCH rc=$?"
python -c "
import json; d=json.load(open('$OUT/bench_default.json'))
print('value %.4g ms %.2f frac %.3f l2 %.3f e2e %.4g clocks %s' % (d['value'], d['ms_per_step'], d['roofline']['frac'], d['l2_red_roofline']['frac'], d['e2e']['value'], d['clocks']))
for k,v in d['extra_configs'].items(): print(' ', k, '%.2f ms' % v.get('kernel_ms',0), 'hbm %.3f' % v.get('hbm_roofline_frac',0), 'l2 %.3f' % (v.get('l2_red_frac') or 0))
"
timeout 600 python bench.py --impl reference --steps 2 --warmup 1 > $OUT/bench_reference.log 2>&1; echo "REFERENCE rc=$?"
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file $OUT/launches_csp.csv python bench.py --steps 2 --warmup 1 --no-cpu-baseline --no-e2e --no-extras > $OUT/ncu_launch.log 2>&1
for cm in csp:history csp:event scatter:history stream:history; do
  c=${cm%%:*}; m=${cm##*:}
  if [ $m = event ]; then K=regex:ev_loop; N=1; else K=regex:history; N=2; fi
  timeout 900 ncu --set full --clock-control none --import-source on -k $K -c $N -o $OUT/prof_${c}_$m python bench.py --config $c --mode $m --steps 1 --warmup 0 --no-cpu-baseline --no-e2e --no-extras > $OUT/ncu_${c}_$m.log 2>&1
  python scripts/ncu_summary.py $OUT/prof_${c}_$m.ncu-rep $OUT/ncu_${c}_$m.md --traffic-key $c/$m > /dev/null 2>&1
  rm -f $OUT/prof_${c}_$m.ncu-rep
done
ls $OUT
