#!/bin/bash
# ncu --set full of the LJ store kernels of one timed slide (validate, apply+restore, one radix scatter)
OUT=gpurun_out/pst; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
B="--steps 2 --warmup 3 --no-cpu-baseline --no-e2e --no-multi-source"
for k in k_store_validate k_apply_restore k_rs_scatter k_heads; do
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:$k -s 4 -c 1 -o $OUT/$k python bench.py $B > $OUT/$k.out 2>&1; echo "$k rc=$?"
done
