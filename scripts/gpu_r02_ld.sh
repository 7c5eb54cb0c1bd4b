# A/B: refill issues the state loads with the status load (ld = working tree) vs HEAD (old)
bash scripts/dev/ab_variants.sh r02_ld "old ld" "scatter:history csp:history split:history stream:history" 2
