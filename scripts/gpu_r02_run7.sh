OUT=gpurun_out/r02_t7; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
NT_PARITY_REPORT=$OUT/parity timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider -x > $OUT/pytest_gpu.log 2>&1
echo "PYTEST $(tail -1 $OUT/pytest_gpu.log)"; grep -E "^FAILED|Error" $OUT/pytest_gpu.log | head -10
bash scripts/dev/ab_variants.sh r02_ab4_blkskip "evpair hnoskip" "csp:history stream:history split:history scatter:history" 2
bash scripts/dev/ab_variants.sh r02_ab5_evqueue "evpair evcomp" "csp:event stream:event split:event scatter:event" 2
