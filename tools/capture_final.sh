#!/bin/bash
# Final-build evidence on one B200 (run under gpurun from the repo root): the
# default bench line, the bench's launch list (ncu gpu__time_duration pass of
# a short no-extras run, after the same command ran clean), and ncu --set full
# captures of the main kernels, exported on the box as raw CSV (plain and
# mangled kernel names) for tools/ncu_csv_summary.py.
O=gpurun_out/final
mkdir -p $O
python bench.py > $O/bench.json 2> $O/bench.err
echo "bench rc=$?" >> $O/status.txt
python bench.py --steps 20 --warmup 3 --no-extras > $O/bench_short.json 2> $O/bench_short.err && \
  ncu --metrics gpu__time_duration.sum --clock-control none -k regex:tdg_ -c 400 --csv \
      --log-file $O/launches_bench.csv python bench.py --steps 20 --warmup 3 --no-extras > /dev/null 2>&1
echo "launches rc=$?" >> $O/status.txt
cap() {
  name=$1; skip=$2; cnt=$3; shift 3
  python tools/ncu_target.py "$@" > /dev/null 2>&1 && \
    timeout 900 ncu --set full --clock-control none --import-source on -k regex:tdg_ -s $skip -c $cnt \
      -o $O/$name python tools/ncu_target.py "$@" > $O/$name.log 2>&1
  echo "$name rc=$?" >> $O/status.txt
  ncu -i $O/$name.ncu-rep --page raw --csv > $O/$name.raw.csv 2>/dev/null
  ncu -i $O/$name.ncu-rep --page raw --csv --print-kernel-base mangled > $O/$name.mangled.csv 2>/dev/null
  [ "$name" = headline ] || rm -f $O/$name.ncu-rep
}
cap headline 1 1 --n 512 --systems 131072
cap pcr 1 1 --n 512 --systems 131072 --algo pcr
cap crpcr256 1 1 --n 512 --systems 131072 --m 256
cap c3rows_f32 1 1 --n 4096 --systems 4096
cap c3rows_f64 1 1 --n 4096 --systems 4096 --dtype f64
cap c3cols_f32 3 3 --n 4096 --systems 4096 --layout cols
cap c5_8192 1 1 --n 8192 --systems 16384
cap large_f32 5 5 --n 1048576 --systems 64
