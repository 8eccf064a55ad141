# usage: bash tools/ab_bench.sh OUT spec...   (A = in-tree build, B = ab/libtridiag_base.so), twice
out=$1; shift
for r in 1 2; do
  python tools/quick_bench.py "$@" | sed 's/^{/{"lib": "new", /' >> $out
  TRIDIAG_LIB_AB=ab/libtridiag_base.so python tools/quick_bench.py "$@" | sed 's/^{/{"lib": "base", /' >> $out
done
