# usage: bash scripts/gpu_ncu_ev.sh TAG CONFIG -- ncu --set full of the persistent event loop
TAG=${1:-evncu}; C=${2:-stream}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 900 ncu --set full --clock-control none --import-source on -k regex:ev_loop -c 1 \
    -o $OUT/prof_${C}_event python bench.py --config $C --mode event --steps 1 --warmup 0 --no-cpu-baseline --no-e2e > $OUT/ncu_${C}_event.log 2>&1
tail -3 $OUT/ncu_${C}_event.log
