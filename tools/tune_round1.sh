#!/bin/bash
# Plan / prefetch / switch-level tuning on one GPU (output: gpurun_out/tune*.jsonl)
cd "$(dirname "$0")/.."
out=gpurun_out/tune1.jsonl; : > $out
for pf in 0 1; do
  for R in 1 2 4 8 16; do
    TRIDIAG_PREFETCH=$pf TRIDIAG_WARP_R=$R timeout 300 python tools/tune.py --dtype f32 --ns 32,64,128,256,512 --algos cr_pcr,cr_rd --ms 2,4,8,16,32 >> $out 2>>gpurun_out/tune1.err
    TRIDIAG_PREFETCH=$pf TRIDIAG_WARP_R=$R timeout 300 python tools/tune.py --dtype f32 --ns 64,128,256,512 --elems 0 --systems 16384 --algos cr_pcr --ms 2,8,32 >> $out 2>>gpurun_out/tune1.err
    TRIDIAG_PREFETCH=$pf TRIDIAG_WARP_R=$R timeout 300 python tools/tune.py --dtype f64 --ns 32,64,128,256,512 --algos cr_pcr,cr_rd --ms 2,4,8,16,32 >> $out 2>>gpurun_out/tune1.err
  done
  TRIDIAG_PREFETCH=$pf timeout 300 python tools/tune.py --dtype f32 --ns 1024,2048,4096,8192 --algos cr,cr_pcr --ms 0,16,32 >> $out 2>>gpurun_out/tune1.err
  TRIDIAG_PREFETCH=$pf timeout 300 python tools/tune.py --dtype f64 --ns 512,1024,2048,4096 --algos cr,cr_pcr --ms 0,16,32 >> $out 2>>gpurun_out/tune1.err
done
wc -l $out
