# round evidence + the XS table-size sweep (direct rows) on scatter
TAG=${1:-r02_final2}
bash scripts/gpu_r02_final.sh $TAG
OUT=gpurun_out/$TAG
for n in 4096 65536 1048576; do
  for x in 0 3; do
    python bench.py --config scatter --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --no-extras --table-size $n \
      --xs-search $x --json-out $OUT/b_scatter_tab${n}_xs$x.json > /dev/null 2>&1
    python -c "
import json; d=json.load(open('$OUT/b_scatter_tab${n}_xs$x.json'))
print('TABLE $n xs=$x kernel_ms %.3f' % d['roofline']['kernel_ms'])" 2>&1 | tail -1
  done
done
