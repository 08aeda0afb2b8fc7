#!/bin/bash
# Build / bench experiment variants of libtds (compile-time switches), side by side.
#   scripts/variant.sh build NAME "-DFLAG=1 ..." unit1 [unit2 ...]   # here: build/var/NAME/libtds.so
#   scripts/variant.sh run NAME "bench args" OUT                       # GPU box: bench with that library
# Only the listed translation units are recompiled; the rest are the product objects.
set -u
ROOT=$(cd "$(dirname "$0")/.." && pwd)
CSRC=$ROOT/paper_conf_ipps_davidsonzo11_b200/csrc
NVCC=${NVCC:-/usr/local/cuda/bin/nvcc}
ARCH="-gencode arch=compute_100a,code=sm_100a"
FLAGS="-O3 -std=c++17 -lineinfo $ARCH -Xcompiler -fPIC"
cmd=$1; name=$2; shift 2
V=$ROOT/build/var/$name
case "$cmd" in
build)
    defs=$1; shift
    make -C "$CSRC" -j8 >/dev/null || exit 1
    mkdir -p "$V/o"
    objs=""
    for f in "$ROOT"/build/csrc/*.o; do
        b=$(basename "$f" .o)
        if [[ " $* " == *" $b "* ]]; then
            $NVCC $FLAGS $defs -c "$CSRC/$b.cu" -o "$V/o/$b.o" -Xptxas -v 2> "$V/o/$b.ptxas.txt" &
            objs="$objs $V/o/$b.o"
        else
            objs="$objs $f"
        fi
    done
    wait
    $NVCC -shared $ARCH -o "$V/libtds.so" $objs -cudart static && echo "built $V/libtds.so" ;;
run)
    args=$1; out=$2
    W=/tmp/tds_var_$name
    rm -rf "$W"; mkdir -p "$W"
    (cd "$ROOT" && tar --exclude=./build --exclude=./gpurun_out --exclude=./.git -cf - .) | (cd "$W" && tar xf -)
    cp "$V/libtds.so" "$W/paper_conf_ipps_davidsonzo11_b200/libtds.so"
    (cd "$W" && timeout 600 python bench.py $args) > "$out" 2> "$out.err"
    echo "$name: $(python -c "import json,sys; d=json.loads(open('$out').read().strip().splitlines()[-1]); print(round(d['ms_per_step'],4), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])" 2>&1)" ;;
*) echo "usage"; exit 2 ;;
esac
