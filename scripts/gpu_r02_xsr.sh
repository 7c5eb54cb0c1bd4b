OUT=gpurun_out/r02_xsr; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -k "xs" > $OUT/pytest.log 2>&1
echo "PYTEST $(tail -1 $OUT/pytest.log)"; grep -E "^FAILED|assert" $OUT/pytest.log | head -8
