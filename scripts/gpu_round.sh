set -x
mkdir -p gpurun_out/r01
python -c "import __graft_entry__ as g; g.build()"
python bench.py --json-out gpurun_out/r01/bench_csp.json 2>&1 | tail -3
for c in stream scatter split; do python bench.py --config $c --no-cpu-baseline --no-e2e --steps 5 --json-out gpurun_out/r01/bench_$c.json 2>&1 | tail -2; done
ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/r01/launches_csp.csv python bench.py --steps 2 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/r01/ncu_launch_bench.log 2>&1
ncu --set full --clock-control none --import-source on -k regex:history -s 1 -c 1 -o gpurun_out/r01/prof_csp_history python bench.py --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > gpurun_out/r01/ncu_full.log 2>&1
ls -la gpurun_out/r01
