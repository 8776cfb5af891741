# L2 eviction-priority variants of the per-edge R / d_out accesses (no persisting window on these sets)
mkdir -p gpurun_out/keep
for lib in build/variants/libppr_keep_*.so; do
  name=$(basename $lib .so)
  for cfg in "tw --workload twitter" "s0of8 --sources 256 --mode shared --shard 0/8" "s256 --sources 256 --mode shared" "lj" "ork --workload orkut"; do
    set -- $cfg; tag=$1; shift
    PPR_LIB=$PWD/$lib timeout 600 python bench.py --steps 5 --warmup 3 --no-cpu-baseline --no-e2e "$@" > gpurun_out/keep/${name}_$tag.json 2> gpurun_out/keep/${name}_$tag.err
    python -c "import json;d=json.load(open('gpurun_out/keep/${name}_$tag.json'));x=d['detail'];print('$name $tag', 'step %.3f push %.3f' % (d['ms_per_step'], x['ms_push']))" 2>/dev/null || { echo "$name $tag failed"; tail -2 gpurun_out/keep/${name}_$tag.err; }
  done
done
