#!/bin/bash
# hot-line microbenchmark + A/B of build/variants (under gpurun)
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 120 ./tools/hotline_bench > gpurun_out/hotline.txt 2>&1; cat gpurun_out/hotline.txt
for rep in 1 2; do bash tools/ab_variants.sh; done
