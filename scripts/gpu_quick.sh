# usage: bash scripts/gpu_quick.sh TAG  -- tests + default benches of the 4 configs
TAG=${1:-quick}
OUT=gpurun_out/$TAG
mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 900 python -m pytest tests -m gpu -x -q -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1
tail -3 $OUT/pytest_gpu.log
for c in csp stream scatter split; do
  python bench.py --config $c --no-cpu-baseline --no-e2e --steps 5 --json-out $OUT/bench_$c.json > /dev/null 2>&1
done
for f in $OUT/bench_*.json; do python -c "
import json; d=json.load(open('$f')); r=d['roofline']
print('$f'.split('/')[-1], f\"value={d['value']:.3e} kernel_ms={r['kernel_ms']:.2f} frac={r['frac']:.3f} clocks={d['clocks']['sm_mhz']}\")"; done
