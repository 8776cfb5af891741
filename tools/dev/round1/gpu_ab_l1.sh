#!/bin/bash
# A/B of the L1 load-policy variants (build/variants) + ncu of the SHARED push at S=32 (shard) and S=256
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
for rep in 1 2; do bash tools/ab_variants.sh; done
for lib in build/variants/libppr_a_base.so build/variants/libppr_c_poolna_doutel.so; do
  name=$(basename $lib .so)
  PPR_LIB=$PWD/$lib timeout 300 python bench.py --sources 256 --shard 0/8 --mode shared --steps 5 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ab_ms_$name.json 2>/dev/null
  python -c "import json;d=json.load(open('gpurun_out/ab_ms_$name.json'));print('ms s0of8 $name', d['ms_per_step'])"
done
timeout 600 ncu --set full --clock-control none -k regex:k_push_ms -s 3 -c 1 -o gpurun_out/prof_ms32 python bench.py --sources 256 --shard 0/8 --mode shared --steps 1 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_ms32.log 2>&1; echo ncu32 rc=$?
timeout 900 ncu --set full --clock-control none -k regex:k_push_ms -s 3 -c 1 -o gpurun_out/prof_ms256 python bench.py --sources 256 --mode shared --steps 1 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_ms256.log 2>&1; echo ncu256 rc=$?
