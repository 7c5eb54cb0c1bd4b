# usage: bash scripts/gpu_ncu_event.sh TAG CONFIG -- ncu --set full of the event-mode kernels mid-run
# (NT_EVENT_HOST_LOOP=1: ncu cannot profile kernels inside a conditional CUDA graph)
TAG=$1; C=${2:-csp}
OUT=gpurun_out/$TAG
mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
NT_EVENT_HOST_LOOP=1 timeout 600 python bench.py --config $C --mode event --steps 2 --warmup 1 --no-cpu-baseline --no-e2e --json-out $OUT/bench_${C}_event_hostloop.json > /dev/null 2>&1
tail -c 400 $OUT/bench_${C}_event_hostloop.json
NT_EVENT_HOST_LOOP=1 ncu --set full --clock-control none --import-source on -k regex:ev_ -s 3000 -c 4 \
    -o $OUT/prof_${C}_event python bench.py --config $C --mode event --steps 1 --warmup 0 --no-cpu-baseline --no-e2e \
    > $OUT/ncu_${C}_event.log 2>&1
tail -3 $OUT/ncu_${C}_event.log
