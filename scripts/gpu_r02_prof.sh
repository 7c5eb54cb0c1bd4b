# usage: bash scripts/gpu_r02_prof.sh TAG "cfg:mode cfg:mode ..." [pytest] -- optional GPU tests, bench lines,
# ncu --set full of the tracking kernel per case (summarised on the box; reports removed)
TAG=${1:-r02prof}; CASES=${2:-"csp:event scatter:history"}; TESTS=${3:-}
OUT=gpurun_out/$TAG
mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
if [ -n "$TESTS" ]; then
  NT_PARITY_REPORT=$OUT/parity timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider -s --durations=10 > $OUT/pytest_gpu.log 2>&1
  tail -1 $OUT/pytest_gpu.log | sed "s/^/PYTEST: /"
  grep -E "^FAILED" $OUT/pytest_gpu.log | head -20 | cut -c1-200
fi
for cm in $CASES; do
  c=${cm%%:*}; m=${cm##*:}
  timeout 300 python bench.py --config $c --mode $m --no-cpu-baseline --no-e2e --steps 3 --json-out $OUT/bench_${c}_$m.json > $OUT/bench_${c}_$m.log 2>&1
  python -c "
import json; d=json.load(open('$OUT/bench_${c}_$m.json')); r=d['roofline']
print('$c $m', f\"value={d['value']:.3e} ms={d['ms_per_step']:.2f} frac={r['frac']:.3f} clocks={d['clocks']['sm_mhz']}\")" 2>&1 | tail -1
done
for cm in $CASES; do
  c=${cm%%:*}; m=${cm##*:}
  if [ $m = event ]; then K=regex:ev_loop; N=1; else K=regex:history; N=2; fi
  timeout 900 ncu --set full --clock-control none --import-source on -k $K -c $N \
      -o $OUT/prof_${c}_$m python bench.py --config $c --mode $m --steps 1 --warmup 0 --no-cpu-baseline --no-e2e > $OUT/ncu_${c}_$m.log 2>&1
  python scripts/ncu_summary.py $OUT/prof_${c}_$m.ncu-rep $OUT/ncu_${c}_$m.md > /dev/null 2>&1
  rm -f $OUT/prof_${c}_$m.ncu-rep
done
ls $OUT
