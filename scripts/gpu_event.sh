# usage: bash scripts/gpu_event.sh TAG -- GPU tests, then event-mode benches of the 4 configs
TAG=${1:-event}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 900 python -m pytest tests -m gpu -x -q -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1
tail -3 $OUT/pytest_gpu.log
grep -m3 -B2 -A30 "Error\|FAILED\|assert" $OUT/pytest_gpu.log | head -80
for c in ${CONFIGS:-csp stream scatter split}; do
  timeout 300 python bench.py --config $c --mode event --no-cpu-baseline --no-e2e --steps 3 --json-out $OUT/bench_${c}_event.json > $OUT/bench_${c}_event.log 2>&1
  python -c "import json; d=json.load(open('$OUT/bench_${c}_event.json')); print('$c event', '%.3e ev/s' % d['value'], '%.2f ms' % d['ms_per_step'])" 2>&1 | tail -1
done
