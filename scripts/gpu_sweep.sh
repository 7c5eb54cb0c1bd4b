# usage: bash scripts/gpu_sweep.sh TAG   (runs on the GPU box)
set -x
TAG=${1:-sweep}
OUT=gpurun_out/$TAG
mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 900 python -m pytest tests -m gpu -x -q -p no:cacheprovider 2>&1 | tail -5
for c in csp stream scatter split; do
  for k in 4 3; do
    python bench.py --config $c --ctas-per-sm $k --no-cpu-baseline --no-e2e --steps 5 --json-out $OUT/bench_${c}_k$k.json > /dev/null 2>&1
  done
done
for r in 4 8 16; do
  python bench.py --config scatter --refill-min $r --no-cpu-baseline --no-e2e --steps 5 --json-out $OUT/bench_scatter_r$r.json > /dev/null 2>&1
done
ls $OUT
