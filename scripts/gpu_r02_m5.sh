# A/B: default kernel compiled for 5 CTAs/SM (96 registers, no spills) vs 6 (80)
bash scripts/dev/ab_variants.sh r02_m5 "base m5" "csp:history stream:history split:history scatter:history" 2
