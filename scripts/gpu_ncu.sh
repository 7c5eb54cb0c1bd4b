# usage: bash scripts/gpu_ncu.sh TAG "config:args" ...   (runs on the GPU box)
TAG=$1; shift
OUT=gpurun_out/$TAG
mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
for spec in "$@"; do
  c=${spec%%:*}; args=${spec#*:}; [ "$args" = "$spec" ] && args=""
  name=$(echo "${c}_${args}" | tr ' -' '__')
  ncu --set full --clock-control none --import-source on -k regex:history -s 1 -c 1 \
      -o $OUT/prof_$name python bench.py --config $c $args --steps 1 --warmup 1 --no-cpu-baseline --no-e2e \
      > $OUT/ncu_$name.log 2>&1
  tail -2 $OUT/ncu_$name.log
done
ls -la $OUT
