# resume ring A/B 2: phase-2 events per vote (NT_P2_INNER) with the ring vs no ring.
TAG=${1:-r02_ring2}
OUT=gpurun_out/$TAG; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
NT_P2_INNER=16 timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -x -k "resume_prefetch or smoke" > $OUT/pytest.log 2>&1
echo "PYTEST(inner2=16) $(tail -1 $OUT/pytest.log)"
for rep in 1 2; do
  for c in csp split scatter; do
    for v in "0 0" "1 0" "1 64" "1 32" "1 16" "1 8" "1 4"; do
      set -- $v
      NT_P2_INNER=$2 python bench.py --config $c --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --no-extras \
        --resume-prefetch $1 --json-out $OUT/b_${c}_rp$1_in$2_r$rep.json > /dev/null 2>&1
      python -c "
import json; d=json.load(open('$OUT/b_${c}_rp$1_in$2_r$rep.json'))
print('$c rp=$1 inner2=$2 rep=$rep', 'kernel_ms %.3f' % d['roofline']['kernel_ms'])" 2>&1 | tail -1
    done
  done
done
