# DEV A/B: tail repacking (NT_TAIL_REPACK = lanes) -> launch 1b; parity first
TAG=${1:-r02_tr}
OUT=gpurun_out/$TAG; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
NT_TAIL_REPACK=16 timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -p no:cacheprovider -x -k "deterministic or production or deferral or two_steps" > $OUT/pytest.log 2>&1
echo "PYTEST(repack 16) $(tail -1 $OUT/pytest.log)"; grep -E "^FAILED" $OUT/pytest.log | head -3
for rep in 1 2; do
  for c in csp split stream scatter; do
    for v in 0 8 16 24 30; do
      NT_TAIL_REPACK=$v python bench.py --config $c --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --no-extras \
        --json-out $OUT/b_${c}_tr${v}_r$rep.json > /dev/null 2>&1
      python -c "
import json; d=json.load(open('$OUT/b_${c}_tr${v}_r$rep.json'))
print('$c repack=$v rep=$rep', 'kernel_ms %.3f' % d['roofline']['kernel_ms'], 'launches', d['gpu_launches'])" 2>&1 | tail -1
    done
  done
done
