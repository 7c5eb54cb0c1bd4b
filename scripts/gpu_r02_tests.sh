# usage: bash scripts/gpu_r02_tests.sh TAG -- GPU test suite (incl. full-scale parity with per-case reports) + smoke
TAG=${1:-r02}
OUT=gpurun_out/$TAG
mkdir -p $OUT
nproc > $OUT/nproc.txt; lscpu | grep -E "Model name|^CPU\(s\)" >> $OUT/nproc.txt
python -c "import __graft_entry__ as g; g.build()"
NT_PARITY_REPORT=$OUT/parity timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider -s --durations=25 > $OUT/pytest_gpu.log 2>&1
tail -3 $OUT/pytest_gpu.log | sed "s/^/PYTEST: /"
grep -E "FAILED|Error" $OUT/pytest_gpu.log | head -20
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke.log 2>&1; echo "SMOKE rc=$?: $(tail -1 $OUT/smoke.log)"
python bench.py --no-cpu-baseline --json-out $OUT/bench_csp.json > $OUT/bench_csp.log 2>&1; tail -c 400 $OUT/bench_csp.log
