# usage: bash scripts/gpu_runs.sh TAG "config args..." ...   (GPU box) -- pytest -m gpu (unless
# NOTEST=1), then one bench line per spec, saved as gpurun_out/TAG/<n>.json and summarised.
TAG=$1; shift
OUT=gpurun_out/$TAG
mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
if [ -z "$NOTEST" ]; then
  timeout 1200 python -m pytest tests -m gpu -x -q -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1
  tail -1 $OUT/pytest_gpu.log | sed "s/^/PYTEST: /"
fi
i=0
for spec in "$@"; do
  i=$((i+1))
  c=${spec%% *}; args=${spec#"$c"}
  timeout 600 python bench.py --config $c $args --no-cpu-baseline --no-e2e --steps ${STEPS:-3} --json-out $OUT/$i.json > $OUT/$i.log 2>&1
  python -c "
import json,sys
try:
  d=json.load(open('$OUT/$i.json')); r=d['roofline']
  print('%-40s %.3e ev/s  %8.2f ms  kern %8.2f ms  frac %.3f  sm %s' % ('$spec', d['value'], d['ms_per_step'], r['kernel_ms'], r['frac'], d['clocks']['sm_mhz']))
except Exception as e: print('$spec FAILED', e); print(open('$OUT/$i.log').read()[-800:])"
done
