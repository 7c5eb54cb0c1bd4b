# A/B: ledger REDs at history end (rl = working tree) vs HEAD (old)
bash scripts/dev/ab_variants.sh r02_rl "old rl" "scatter:history scatter:event csp:history split:history csp:event" 2
