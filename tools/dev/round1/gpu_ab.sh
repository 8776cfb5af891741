#!/bin/bash
# A/B of build/variants/*.so on the LJ bench, plus optional extra args via BENCH_ARGS
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
for rep in 1 2; do bash tools/ab_variants.sh; done
