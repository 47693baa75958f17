#!/bin/bash
# Build a variant of libchol_b200.so with extra nvcc flags into variants/<name>.so
# (A/B experiments, CHOL_LIB_OVERRIDE=variants/<name>.so); usage: tools/build_variant.sh name [flags...]
set -e
name=$1; shift
cd "$(dirname "$0")/.."
mkdir -p variants/obj_$name
CS=paper_conf_ipps_agullobehkmt15_b200/csrc
F="-O3 -std=c++17 -gencode arch=compute_100a,code=sm_100a -lineinfo -Xcompiler -fPIC -Xcompiler -O2 --expt-relaxed-constexpr $@"
for s in api.cu kernels.cu sched.cu solve.cu dag.cpp sim.cpp hetero.cpp; do
  nvcc $F -c $CS/$s -o variants/obj_$name/${s%.*}.o &
done
wait
nvcc -shared -gencode arch=compute_100a,code=sm_100a -o variants/$name.so variants/obj_$name/*.o
echo variants/$name.so
