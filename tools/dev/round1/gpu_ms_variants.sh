# SHARED push tile-size variants (build/variants/libppr_*.so) on the 8-GPU rank shard and the 256-source handle
mkdir -p gpurun_out/msvar
for lib in build/variants/libppr_*.so; do
  name=$(basename $lib .so)
  for cfg in "s0of8 --shard 0/8" "s3of8 --shard 3/8" "s256"; do
    set -- $cfg; tag=$1; shift
    PPR_LIB=$PWD/$lib timeout 600 python bench.py --sources 256 --mode shared --steps ${STEPS:-5} --warmup 3 --no-cpu-baseline --no-e2e "$@" > gpurun_out/msvar/${name}_$tag.json 2> gpurun_out/msvar/${name}_$tag.err
    python -c "import json;d=json.load(open('gpurun_out/msvar/${name}_$tag.json'));x=d['detail'];print('$name $tag', 'step %.3f push %.3f' % (d['ms_per_step'], x['ms_push']))" 2>/dev/null || { echo "$name $tag failed"; tail -2 gpurun_out/msvar/${name}_$tag.err; }
  done
done
for cfg in "s0of8 --shard 0/8" "s3of8 --shard 3/8" "s256"; do
  set -- $cfg; tag=$1; shift
  for w in default nowin; do
    [ $w = nowin ] && export PPR_L2_PERSIST=0 || unset PPR_L2_PERSIST
    timeout 600 python bench.py --sources 256 --mode shared --steps ${STEPS:-5} --warmup 3 --no-cpu-baseline --no-e2e "$@" > gpurun_out/msvar/${w}_$tag.json 2> gpurun_out/msvar/${w}_$tag.err
    python -c "import json;d=json.load(open('gpurun_out/msvar/${w}_$tag.json'));x=d['detail'];print('$w $tag', 'step %.3f push %.3f' % (d['ms_per_step'], x['ms_push']))" 2>/dev/null || { echo "$w $tag failed"; tail -2 gpurun_out/msvar/${w}_$tag.err; }
  done
done
unset PPR_L2_PERSIST
PPR_L2_PERSIST=0 timeout 600 python bench.py --workload orkut --steps 10 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/msvar/ork_nowin.json 2>/dev/null; python -c "import json;d=json.load(open('gpurun_out/msvar/ork_nowin.json'));print('ork nowin push %.3f' % d['detail']['ms_push'])"
PPR_L2_PERSIST=0 timeout 600 python bench.py --steps 30 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/msvar/lj_nowin.json 2>/dev/null; python -c "import json;d=json.load(open('gpurun_out/msvar/lj_nowin.json'));print('lj nowin push %.3f' % d['detail']['ms_push'])"
