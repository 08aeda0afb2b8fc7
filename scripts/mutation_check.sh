#!/bin/bash
# Mutation check of the coupling tests ("a debug build that
# zeroes the top-row coupling makes the new tests fail").
#
#   scripts/mutation_check.sh build      # here (CPU): libtds_mut{1..7}.so under build/mut/
#   scripts/mutation_check.sh run OUT    # on the GPU box: run tests/test_coupling.py against each
#
# Each mutant is the product library with ONE long-range coupling term
# dropped (csrc/common.cuh TDS_MUTATE sites 1-7); only the four on-chip
# translation units are recompiled, the rest are the product objects.
set -u
ROOT=$(cd "$(dirname "$0")/.." && pwd)
CSRC=$ROOT/paper_conf_ipps_davidsonzo11_b200/csrc
MUT=$ROOT/build/mut
NVCC=${NVCC:-/usr/local/cuda/bin/nvcc}
ARCH="-gencode arch=compute_100a,code=sm_100a"
FLAGS="-O3 -std=c++17 -lineinfo $ARCH -Xcompiler -fPIC"
SITES="${SITES:-1 2 3 4 5 6 7}"
case "${1:-}" in
build)
    make -C "$CSRC" -j8 >/dev/null || exit 1
    for k in $SITES; do
        mkdir -p "$MUT/o$k"
        objs=""
        for f in "$ROOT"/build/csrc/*.o; do
            b=$(basename "$f" .o)
            case $b in
            onchip|onchip_pipe|onchip_cpipe|onchip_coalesced)
                $NVCC $FLAGS -DTDS_MUTATE=$k -c "$CSRC/$b.cu" -o "$MUT/o$k/$b.o" &
                objs="$objs $MUT/o$k/$b.o" ;;
            *) objs="$objs $f" ;;
            esac
        done
        wait
        $NVCC -shared $ARCH -o "$MUT/libtds_mut$k.so" $objs -cudart static || exit 1
        echo "built $MUT/libtds_mut$k.so"
    done ;;
run)
    OUT=${2:-$ROOT/gpurun_out/mutation}
    mkdir -p "$OUT"
    for k in $SITES; do
        W=/tmp/tds_mut$k
        rm -rf "$W"; mkdir -p "$W"
        (cd "$ROOT" && tar --exclude=./build --exclude=./gpurun_out --exclude=./.git -cf - .) | (cd "$W" && tar xf -)
        cp "$MUT/libtds_mut$k.so" "$W/paper_conf_ipps_davidsonzo11_b200/libtds.so"
        (cd "$W" && timeout 900 python -m pytest tests/test_coupling.py -m gpu -q -p no:cacheprovider \
            -o addopts="" 2>&1 | tail -60) > "$OUT/mut$k.log"
        echo "mutant $k: $(grep -E '[0-9]+ (passed|failed)' "$OUT/mut$k.log" | tail -1)"
    done ;;
*) echo "usage: $0 build | run [outdir]"; exit 2 ;;
esac
