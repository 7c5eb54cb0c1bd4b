# usage: bash scripts/gpu_prof.sh TAG   -- launch list of the default bench + ncu full of csp/stream history
TAG=${1:-prof}
OUT=gpurun_out/$TAG
mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file $OUT/launches_csp.csv \
    python bench.py --steps 2 --warmup 1 --no-cpu-baseline --no-e2e > $OUT/ncu_launch_bench.log 2>&1
bash scripts/gpu_ncu.sh $TAG csp stream ${EXTRA_CFGS}
