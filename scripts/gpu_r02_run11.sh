OUT=gpurun_out/r02_t11; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
NT_PARITY_REPORT=$OUT/parity timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1
echo "PYTEST $(tail -1 $OUT/pytest_gpu.log)"; grep -E "^FAILED|Error" $OUT/pytest_gpu.log | head -10
bash scripts/dev/ab_variants.sh r02_ab9_facet2_clobber "f2c0 f2c1 f1c0 f1c1" "csp:event stream:event split:event scatter:event csp:history split:history" 2 | grep -v pytest
