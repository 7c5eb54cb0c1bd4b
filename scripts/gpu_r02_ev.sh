# usage: bash scripts/gpu_r02_ev.sh TAG -- tests + event/history bench lines on csp/stream/scatter/split
TAG=${1:-r02ev}
OUT=gpurun_out/$TAG
mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
NT_PARITY_REPORT=$OUT/parity timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider -s --durations=25 > $OUT/pytest_gpu.log 2>&1
tail -1 $OUT/pytest_gpu.log | sed "s/^/PYTEST: /"
grep -E "^FAILED" $OUT/pytest_gpu.log | head -20 | cut -c1-200
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke.log 2>&1; echo "SMOKE rc=$?: $(tail -1 $OUT/smoke.log)"
for c in csp stream scatter split; do
  for m in event history; do
    timeout 300 python bench.py --config $c --mode $m --no-cpu-baseline --no-e2e --steps 3 --json-out $OUT/bench_${c}_$m.json > $OUT/bench_${c}_$m.log 2>&1
    python -c "
import json; d=json.load(open('$OUT/bench_${c}_$m.json')); r=d['roofline']
print('$c $m', f\"value={d['value']:.3e} ms={d['ms_per_step']:.2f} frac={r['frac']:.3f} clocks={d['clocks']['sm_mhz']}\")" 2>&1 | tail -1
  done
done
